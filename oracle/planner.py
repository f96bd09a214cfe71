"""Brute-force oracle for the paper's data-management framework (sp_plan_buffers).

TEST INFRASTRUCTURE ONLY — see oracle/__init__.py.  Shares no code with the product
planner (paper_conf_ppopp_baskaranbkrrs08_b200/csrc/planner.cpp).

Follows P = /root/reference/PAPER.md §2-§3 step by step, by enumeration of integer
points (the method reaches exactly this result, so the plain definition is the oracle):

1. statement domains: the integer points of an explicit enumeration box (supplied by
   the test generator) that satisfy every row r . (i, p, 1) >= 0          (§2)
2. data space of a reference: the image {F . (i, p, 1)} of its statement's domain
                                                                            (§2)
3. per array, partitions of the data spaces:
   * PER_ARRAY  — one partition holding every reference (Figure 1, P:L498-556;
     DESIGN.md reading R-P1),
   * COMPONENTS — connected components of the overlap graph (edge iff the two data
     spaces intersect)                                      (Alg. 2 step 5)
4. per partition: lb_k / ub_k = min / max of coordinate k over the union of its data
   spaces; size = prod(ub_k - lb_k + 1)                     (Alg. 2 steps 7-9)
   local access of each ref = F with its constant column minus g = lb
   move-in set = union of the read data spaces, move-out set = union of the write data
   spaces; their bounding boxes and cardinalities
5. V_in = sum over connected components of the read data spaces of their bounding-box
   volume; V_out likewise for writes
6. Algorithm 1 (Cond. (1) P:L333-334, delta P:L344-345): beneficial iff some
   ref has rank(F restricted to iterator columns) < depth of its statement; otherwise
   iff sum over pairs of |D_r ∩ D_r'| > delta * |∪ D_r|      (readings R-P3, R-P4)
7. compress (§3.1.2; reading R-P8): the local array has the dimensions of the
   convex hull of the partition's data spaces.  Dimension k is left out when, on the set
   of points, it is an affine function of the dimensions before it — i.e. when the
   difference vectors p - p0 (p0 the first point) have the same rank restricted to the
   first k+1 coordinates as to the first k.  size = prod over the kept k of
   (ub_k - lb_k + 1); the local access function F' drops the other rows (given as zero
   rows: local index 0 along an extent-1 axis).

Buffers are listed ordered by (array id, smallest ref index in the partition).
With reuse_filter, partitions that are not beneficial are not staged: they are not
listed and their refs map to -1 (GPUs stage only beneficial partitions).
"""
from __future__ import annotations

import itertools
from fractions import Fraction

import numpy as np

PER_ARRAY = 0
COMPONENTS = 1

OK = 0
ERR_INVALID_ARG = -1
ERR_UNBOUNDED = -2
ERR_CAPACITY = -3
ERR_OVERFLOW = -4
ERR_UNSUPPORTED = -5
ERR_SMEM_LIMIT = -6

INT64_MAX = (1 << 63) - 1


def enumerate_domain(stmt: dict, params: list[int], box: list[tuple[int, int]]) -> np.ndarray:
    """All integer points of `box` satisfying the statement's rows; int64 [n_points, depth]."""
    depth = stmt["depth"]
    if depth == 0:
        pts = np.zeros((1, 0), dtype=np.int64)
    else:
        axes = [np.arange(lo, hi + 1, dtype=np.int64) for lo, hi in box]
        grids = np.meshgrid(*axes, indexing="ij")
        pts = np.stack([g.reshape(-1) for g in grids], axis=1)
    rows = np.asarray(stmt["rows"], dtype=np.int64).reshape(-1, depth + len(params) + 1)
    if rows.shape[0] == 0 or pts.shape[0] == 0:
        return pts
    hom = np.concatenate([pts, np.tile(np.asarray(params + [1], dtype=np.int64), (pts.shape[0], 1))], axis=1)
    keep = np.all(hom @ rows.T >= 0, axis=1)
    return pts[keep]


def data_space(ref: dict, pts: np.ndarray, params: list[int]) -> np.ndarray:
    """Image F . (i, p, 1) of the domain points; unique rows, int64 [n, rank]."""
    rank = ref["rank"]
    F = np.asarray(ref["rows"], dtype=np.int64).reshape(rank, -1)
    if pts.shape[0] == 0:
        return np.zeros((0, rank), dtype=np.int64)
    hom = np.concatenate([pts, np.tile(np.asarray(params + [1], dtype=np.int64), (pts.shape[0], 1))], axis=1)
    img = hom @ F.T
    return np.unique(img, axis=0)


def _as_set(ds: np.ndarray) -> set:
    return set(map(tuple, ds.tolist()))


def exact_rank(M: list[list[int]]) -> int:
    """Rank by exact rational Gaussian elimination."""
    A = [[Fraction(v) for v in row] for row in M]
    if not A:
        return 0
    rows, cols = len(A), len(A[0])
    r = 0
    for c in range(cols):
        piv = next((i for i in range(r, rows) if A[i][c] != 0), None)
        if piv is None:
            continue
        A[r], A[piv] = A[piv], A[r]
        for i in range(rows):
            if i != r and A[i][c] != 0:
                f = A[i][c] / A[r][c]
                A[i] = [a - f * b for a, b in zip(A[i], A[r])]
        r += 1
        if r == rows:
            break
    return r


def _components(sets: list[set]) -> list[list[int]]:
    """Connected components of the overlap graph (edge iff non-empty intersection)."""
    n = len(sets)
    parent = list(range(n))

    def find(x):
        while parent[x] != x:
            parent[x] = parent[parent[x]]
            x = parent[x]
        return x

    for i in range(n):
        for j in range(i + 1, n):
            if sets[i] & sets[j]:
                parent[find(i)] = find(j)
    groups: dict[int, list[int]] = {}
    for i in range(n):
        groups.setdefault(find(i), []).append(i)
    return sorted(groups.values(), key=min)


def _bbox(points: set, rank: int):
    if not points:
        return [0] * rank, [-1] * rank
    arr = np.array(sorted(points), dtype=np.int64).reshape(-1, rank)
    return arr.min(axis=0).tolist(), arr.max(axis=0).tolist()


def _volume(lb, ub) -> int:
    v = 1
    for lo, hi in zip(lb, ub):
        v *= max(0, hi - lo + 1)
    return v


def kept_dims(points: set, rank: int) -> list[int]:
    """Step 7: the dimensions k whose prefix rank of the difference vectors increases."""
    pts = sorted(points)
    if not pts:
        return []
    p0 = pts[0]
    diffs = [[c - c0 for c, c0 in zip(p, p0)] for p in pts[1:]]
    if not diffs:
        return []
    kept, prev = [], 0
    for k in range(rank):
        rk = exact_rank([row[:k + 1] for row in diffs])
        if rk > prev:
            kept.append(k)
        prev = rk
    return kept


def plan_buffers(block: dict, mode: int = PER_ARRAY, delta: float = 0.30, reuse_filter: bool = False,
                 mup_elems: int = 0, compress: bool = False) -> dict:
    """Oracle plan.  block = {"params": [...], "stmts": [{"depth", "rows", "box"}],
    "refs": [{"stmt", "array", "is_write", "rank", "rows"}]}.  Returns
    {"status", "buffers": [...], "ref_buf": [...], "local_rows": [[...]...]}."""
    params = list(block.get("params", []))
    stmts = block["stmts"]
    refs = block["refs"]
    P = len(params)
    doms = [enumerate_domain(s, params, s["box"]) for s in stmts]
    spaces = [data_space(r, doms[r["stmt"]], params) for r in refs]
    sets = [_as_set(s) for s in spaces]

    arrays = sorted({r["array"] for r in refs})
    parts: list[tuple[int, list[int]]] = []
    for a in arrays:
        ids = [k for k, r in enumerate(refs) if r["array"] == a]
        if mode == PER_ARRAY:
            parts.append((a, ids))
        else:
            for comp in _components([sets[k] for k in ids]):
                parts.append((a, [ids[c] for c in comp]))
    parts.sort(key=lambda t: (t[0], min(t[1])))

    buffers = []
    ref_buf = [-1] * len(refs)
    for a, ids in parts:
        rank = refs[ids[0]]["rank"]
        union = set().union(*[sets[k] for k in ids])
        lb, ub = _bbox(union, rank)
        size = _volume(lb, ub)
        kept = list(range(rank))
        if compress:
            kept = kept_dims(union, rank)
            if union:
                size = _volume([lb[k] for k in kept], [ub[k] for k in kept])
        rd = [k for k in ids if not refs[k]["is_write"]]
        wr = [k for k in ids if refs[k]["is_write"]]
        in_set = set().union(*[sets[k] for k in rd]) if rd else set()
        out_set = set().union(*[sets[k] for k in wr]) if wr else set()
        in_lb, in_ub = _bbox(in_set, rank)
        out_lb, out_ub = _bbox(out_set, rank)
        v_in = sum(_volume(*_bbox(set().union(*[sets[rd[c]] for c in comp]), rank))
                   for comp in _components([sets[k] for k in rd])) if rd else 0
        v_out = sum(_volume(*_bbox(set().union(*[sets[wr[c]] for c in comp]), rank))
                    for comp in _components([sets[k] for k in wr])) if wr else 0
        # Algorithm 1
        beneficial = False
        for k in ids:
            depth = stmts[refs[k]["stmt"]]["depth"]
            F = np.asarray(refs[k]["rows"], dtype=np.int64).reshape(rank, -1)
            if exact_rank(F[:, :depth].tolist()) < depth:
                beneficial = True
        overlap = 0
        for i, j in itertools.combinations(ids, 2):
            overlap += len(sets[i] & sets[j])
        if not beneficial and overlap > delta * len(union):
            beneficial = True
        buf = {
            "array": a, "rank": rank, "beneficial": int(beneficial), "n_refs": len(ids),
            "lb": lb, "ub": ub, "size": size, "v_in_ub": v_in, "v_out_ub": v_out,
            "in_lb": in_lb, "in_ub": in_ub, "in_count": len(in_set),
            "in_dense": int(len(in_set) == _volume(in_lb, in_ub) and len(in_set) > 0),
            "out_lb": out_lb, "out_ub": out_ub, "out_count": len(out_set),
            "out_dense": int(len(out_set) == _volume(out_lb, out_ub) and len(out_set) > 0),
            "overlap": overlap, "union_count": len(union), "refs": ids,
            "n_dims": len(kept) if (union or not compress) else 0, "kept": kept,
        }
        if reuse_filter and not beneficial:
            continue
        for k in ids:
            ref_buf[k] = len(buffers)
        buffers.append(buf)

    for b in buffers:
        for key in ("size", "v_in_ub", "v_out_ub"):
            if b[key] > INT64_MAX:
                return {"status": ERR_OVERFLOW, "buffers": [], "ref_buf": [], "local_rows": []}
    if mup_elems > 0 and sum(b["size"] for b in buffers) > mup_elems:
        return {"status": ERR_SMEM_LIMIT, "buffers": buffers, "ref_buf": ref_buf, "local_rows": []}

    local_rows = []
    for k, r in enumerate(refs):
        depth = stmts[r["stmt"]]["depth"]
        F = [list(row) for row in np.asarray(r["rows"], dtype=np.int64).reshape(r["rank"], depth + P + 1).tolist()]
        if ref_buf[k] >= 0:
            g = buffers[ref_buf[k]]["lb"]
            for d in range(r["rank"]):
                F[d][-1] -= g[d]
                if d not in buffers[ref_buf[k]]["kept"]:
                    F[d] = [0] * len(F[d])
        local_rows.append(F)
    return {"status": OK, "buffers": buffers, "ref_buf": ref_buf, "local_rows": local_rows}
