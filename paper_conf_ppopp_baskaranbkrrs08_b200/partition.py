"""Host-side decomposition logic of the multi-GPU layer.

* Jacobi: contiguous slabs of the 1-D domain, one per rank, boundaries on multiples of
  4 cells (16-byte aligned TMA copies), each slab at least one halo (H cells) wide so a
  single neighbour supplies a whole halo.
* ME: the flattened (pair, macroblock-row) space split into contiguous ranges balanced by
  the number of valid candidates (edge rows have fewer), plus the reference-frame rows each
  range needs (R-row halo above and below, clipped to the frame).

Pure integer arithmetic; no method arithmetic (no stencil, no SAD).
"""
from __future__ import annotations


def jacobi_slabs(n: int, nranks: int, halo: int) -> list[tuple[int, int]]:
    """[(x_begin, n_local)] for each rank: contiguous, covering [0, n), x_begin % 4 == 0."""
    if nranks < 1:
        raise ValueError("nranks >= 1")
    bounds = [0]
    for r in range(1, nranks):
        b = (n * r // nranks) & ~3
        bounds.append(max(b, bounds[-1]))
    bounds.append(n)
    out = [(bounds[r], bounds[r + 1] - bounds[r]) for r in range(nranks)]
    if nranks > 1 and any(nl < halo for _, nl in out):
        raise ValueError(f"every slab must hold at least one halo ({halo} cells); n={n} is too small for {nranks} ranks")
    return out


def me_valid_dy(y0: int, frame_height: int, search_range: int) -> int:
    """Number of valid vertical displacements of an MB at row y0 (restricted vectors)."""
    return min(search_range, frame_height - 16 - y0) - max(-search_range, -y0) + 1


def me_row_ranges(n_pairs: int, frame_height: int, search_range: int, nranks: int) -> list[tuple[int, int]]:
    """Split the flattened (pair, MB row) index space [0, n_pairs * mby) into nranks
    contiguous ranges [begin, end) balanced by valid-candidate count."""
    mby = frame_height // 16
    w = [me_valid_dy(16 * (k % mby), frame_height, search_range) for k in range(n_pairs * mby)]
    total = sum(w)
    out, acc, begin = [], 0, 0
    for r in range(nranks):
        target = total * (r + 1) / nranks
        end = begin
        while end < len(w) and (acc + w[end] <= target or r == nranks - 1):
            acc += w[end]
            end += 1
        out.append((begin, end))
        begin = end
    return out


def me_band_rows(mb_row_begin: int, mb_row_end: int, frame_height: int, search_range: int) -> tuple[int, int]:
    """Frame rows [row0, row1) a rank must hold to search MB rows [mb_row_begin, mb_row_end):
    the current blocks plus an R-row reference halo above and below, clipped to the frame."""
    row0 = max(0, 16 * mb_row_begin - search_range)
    row1 = min(frame_height, 16 * mb_row_end + search_range)
    return row0, row1


def split_flat_range(begin: int, end: int, mby: int) -> list[tuple[int, int, int]]:
    """Decompose a flat (pair * mby + row) range into per-pair (pair, row_begin, row_end) pieces."""
    out = []
    k = begin
    while k < end:
        p, r = divmod(k, mby)
        e = min(end, (p + 1) * mby)
        out.append((p, r, r + (e - k)))
        k = e
    return out


def me_needed_rows(pieces, f: int, frame_height: int, search_range: int) -> list[tuple[int, int]]:
    """Rows of global frame f that the range `pieces` (split_flat_range output) reads, as sorted
    disjoint intervals [r0, r1): as the reference of pair f (the band rows with the R-row halo,
    me_band_rows) and as the current frame of pair f - 1 (the current blocks' rows).  A range that
    ends inside pair f - 1 and starts pair f needs two separate bands of frame f."""
    iv = []
    for p, r0, r1 in pieces:
        if p == f:  # reference frame of pair p
            iv.append(me_band_rows(r0, r1, frame_height, search_range))
        if p + 1 == f:  # current frame of pair p
            iv.append((16 * r0, 16 * r1))
    out = []
    for a, b in sorted(x for x in iv if x[1] > x[0]):
        if out and a <= out[-1][1]:
            out[-1] = (out[-1][0], max(out[-1][1], b))
        else:
            out.append((a, b))
    return out
