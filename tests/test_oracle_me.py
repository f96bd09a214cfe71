"""Pins for the motion-estimation oracle (oracle/oracle.c spo_me_search).

Readings R-M1..R-M6: Fig. 2 nest with WS = 16,
S1 read as SAD accumulation, candidates [-R, R]^2 restricted to the frame, tie-break
(SAD, |dx|+|dy|, dy, dx).
"""
import numpy as np
import pytest

import oracle
import sp_inputs


def _brute_numpy(ref, cur, W, H, R):
    """Textbook full search written independently with numpy broadcasting."""
    mbx, mby = W // 16, H // 16
    side = 2 * R + 1
    mvs, sads, surf = [], [], []
    for by in range(mby):
        for bx in range(mbx):
            x0, y0 = 16 * bx, 16 * by
            c = cur[y0:y0 + 16, x0:x0 + 16].astype(np.int64)
            S = np.full((side, side), 0xFFFFFFFF, dtype=np.int64)
            for dy in range(-R, R + 1):
                for dx in range(-R, R + 1):
                    if 0 <= x0 + dx and x0 + dx + 16 <= W and 0 <= y0 + dy and y0 + dy + 16 <= H:
                        r = ref[y0 + dy:y0 + dy + 16, x0 + dx:x0 + dx + 16].astype(np.int64)
                        S[dy + R, dx + R] = np.abs(c - r).sum()
            cands = [(S[dy + R, dx + R], abs(dx) + abs(dy), dy, dx)
                     for dy in range(-R, R + 1) for dx in range(-R, R + 1) if S[dy + R, dx + R] != 0xFFFFFFFF]
            best = min(cands)
            mvs.append((best[3], best[2]))
            sads.append(best[0])
            surf.append(S.reshape(-1))
    return np.array(mvs), np.array(sads), np.array(surf)


@pytest.mark.parametrize("W,H,R,gen", [(48, 32, 4, "seq"), (40, 36, 3, "uniform"), (64, 48, 8, "seq"),
                                       (35, 50, 2, "uniform"), (33, 17, 0, "seq")])
def test_matches_numpy_brute_force(W, H, R, gen):
    if gen == "seq":
        fr = sp_inputs.me_sequence(2, W, H, max(R, 2), seed=5)
    else:
        fr = sp_inputs.me_uniform_frames(2, W, H, seed=9)
    ref, cur = fr[0], fr[1]
    mv, sad, surf = oracle.me_search(ref, cur, W, H, R, with_surface=True)
    bmv, bsad, bsurf = _brute_numpy(ref, cur, W, H, R)
    assert np.array_equal(mv, bmv)
    assert np.array_equal(sad, bsad)
    assert np.array_equal(surf.astype(np.int64), bsurf)


def test_identical_frames_zero_motion():
    fr = sp_inputs.me_sequence(1, 96, 64, 8, seed=4)
    mv, sad, _ = oracle.me_search(fr[0], fr[0], 96, 64, 8)
    assert np.all(mv == 0) and np.all(sad == 0)


def test_flat_frames_tie_break():
    # every valid candidate has SAD 256*|c1-c2|; the tie-break picks (0,0)
    ref = np.full((48, 64), 17, dtype=np.uint8)
    cur = np.full((48, 64), 20, dtype=np.uint8)
    mv, sad, surf = oracle.me_search(ref, cur, 64, 48, 5, with_surface=True)
    assert np.all(mv == 0) and np.all(sad == 256 * 3)
    assert set(np.unique(surf).tolist()) <= {256 * 3, 0xFFFFFFFF}


@pytest.mark.parametrize("sx,sy", [(3, -2), (-4, 4), (0, 1)])
def test_shifted_frames_recover_vector(sx, sy):
    W, H, R = 64, 80, 4
    fr = sp_inputs.me_shift_pair(W, H, sx, sy)
    mv, sad, _ = oracle.me_search(fr[0], fr[1], W, H, R)
    k = 0
    for by in range(H // 16):
        for bx in range(W // 16):
            x0, y0 = 16 * bx, 16 * by
            if 0 <= x0 + sx and x0 + sx + 16 <= W and 0 <= y0 + sy and y0 + sy + 16 <= H:
                assert tuple(mv[k]) == (sx, sy) and sad[k] == 0
            k += 1


def _valid_count(W, H, R):
    """Closed form: per MB, (#valid dx) * (#valid dy) with 0 <= x0+dx <= W-16."""
    tot = 0
    for by in range(H // 16):
        y0 = 16 * by
        ny = min(R, H - 16 - y0) - max(-R, -y0) + 1
        for bx in range(W // 16):
            x0 = 16 * bx
            nx = min(R, W - 16 - x0) - max(-R, -x0) + 1
            tot += nx * ny
    return tot


def test_valid_candidate_counts_cif():
    # M2 = CIF 352x288, R = 16: 390,028 valid of 396 * 33^2 = 431,244
    assert _valid_count(352, 288, 16) == 390028
    assert _valid_count(1920, 1080, 32) == 32934600
    fr = sp_inputs.me_sequence(2, 352, 288, 16)
    mv, sad, surf = oracle.me_search(fr[0], fr[1], 352, 288, 16, with_surface=True)
    assert int(np.count_nonzero(surf != 0xFFFFFFFF)) == 390028
    assert sad.max() <= 255 * 256


def test_generator_sequence_counter_based():
    full = sp_inputs.me_sequence(3, 128, 96, 16, seed=11)
    band = sp_inputs.me_frame(2, 128, 96, 16, seed=11, row_begin=40, row_end=70)
    assert np.array_equal(full[2, 40:70], band)
    # consecutive frames are related by motion: away from the frame border (where the true
    # vector may point outside the frame) most macroblocks find a match at noise level
    fr = sp_inputs.me_sequence(3, 352, 288, 16, seed=11)
    mv, sad, _ = oracle.me_search(fr[1], fr[2], 352, 288, 16)
    sad = sad.reshape(18, 22)[2:-2, 2:-2]
    assert np.median(sad) < 256 * 4


# ---- unrestricted motion vectors (N4, reading R-M7) ------------------------------------
def _brute_unrestricted(ref, cur, W, H, R):
    """Independent twin: numpy edge padding (np.pad mode='edge') + broadcast SADs."""
    P = R + 16
    rp = np.pad(ref[:, :W].astype(np.int64), P, mode="edge")
    mvs, sads = [], []
    for by in range(H // 16):
        for bx in range(W // 16):
            x0, y0 = 16 * bx, 16 * by
            c = cur[y0:y0 + 16, x0:x0 + 16].astype(np.int64)
            best = None
            for dy in range(-R, R + 1):
                for dx in range(-R, R + 1):
                    r = rp[P + y0 + dy:P + y0 + dy + 16, P + x0 + dx:P + x0 + dx + 16]
                    k = (int(np.abs(c - r).sum()), abs(dx) + abs(dy), dy, dx)
                    best = k if best is None or k < best else best
            mvs.append((best[3], best[2]))
            sads.append(best[0])
    return np.array(mvs), np.array(sads)


@pytest.mark.parametrize("W,H,R", [(48, 32, 4), (40, 36, 3), (64, 48, 8)])
def test_unrestricted_matches_numpy_edge_padding(W, H, R):
    fr = sp_inputs.me_sequence(2, W, H, max(R, 2), seed=6)
    mv, sad, _ = oracle.me_search(fr[0], fr[1], W, H, R, unrestricted=True)
    bmv, bsad = _brute_unrestricted(fr[0], fr[1], W, H, R)
    assert np.array_equal(mv, bmv) and np.array_equal(sad, bsad)


def test_unrestricted_reduces_to_restricted_inside():
    # interior macroblocks (every candidate inside the frame) give identical results
    W, H, R = 96, 96, 8
    fr = sp_inputs.me_sequence(2, W, H, R, seed=8)
    mv_u, sad_u, _ = oracle.me_search(fr[0], fr[1], W, H, R, unrestricted=True)
    mv_r, sad_r, _ = oracle.me_search(fr[0], fr[1], W, H, R)
    for k in range((W // 16) * (H // 16)):
        bx, by = k % (W // 16), k // (W // 16)
        if 16 * bx - R >= 0 and 16 * bx + 16 + R <= W and 16 * by - R >= 0 and 16 * by + 16 + R <= H:
            assert tuple(mv_u[k]) == tuple(mv_r[k]) and sad_u[k] == sad_r[k]
    # and the unrestricted optimum is never worse
    assert np.all(sad_u <= sad_r)
