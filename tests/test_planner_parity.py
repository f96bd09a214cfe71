"""Product planner (libsp sp_plan_buffers, C++: Fourier-Motzkin scanning + sorted-set
algebra) against the brute-force oracle (oracle/planner.py: box enumeration + Python sets).
Bit-exact on every field: bounds, sizes, move-in/out sets, V_in/V_out, Alg. 1 verdicts,
reference-to-buffer map and local access functions."""
import json
import os
import random

import numpy as np
import pytest

import paper_conf_ppopp_baskaranbkrrs08_b200 as sp
from oracle import planner as O

GOLD = os.path.join(os.path.dirname(__file__), "golden", "figure1.json")
FIELDS = ["array", "rank", "beneficial", "n_refs", "lb", "ub", "size", "v_in_ub", "v_out_ub", "in_lb", "in_ub",
          "in_count", "in_dense", "out_lb", "out_ub", "out_count", "out_dense", "overlap", "union_count",
          "n_dims", "kept"]


def _compare(block, **kw):
    o = O.plan_buffers(block, **kw)
    p = sp.plan_buffers(block, **kw)
    assert p["status"] == o["status"], (p["status"], o["status"])
    if o["status"] != 0:
        return o, p
    assert len(p["buffers"]) == len(o["buffers"])
    for bp, bo in zip(p["buffers"], o["buffers"]):
        for f in FIELDS:
            assert bp[f] == bo[f], (f, bp[f], bo[f])
    assert p["ref_buf"] == o["ref_buf"]
    assert p["local_rows"] == o["local_rows"]
    return o, p


@pytest.mark.parametrize("mode", [O.PER_ARRAY, O.COMPONENTS])
def test_figure1(mode):
    blk = json.load(open(GOLD))["block"]
    _compare(blk, mode=mode)
    _compare(blk, mode=mode, reuse_filter=True)


def _rand_block(rng: random.Random):
    P = rng.randint(0, 2)
    params = [rng.randint(0, 5) for _ in range(P)]
    stmts = []
    for _ in range(rng.randint(1, 3)):
        d = rng.randint(1, 3)
        rows = []
        lo, hi = -6, 9
        for k in range(d):
            # box part keeps the domain inside the oracle's enumeration box
            r = [0] * (d + P + 1)
            r[k] = 1
            r[-1] = -lo
            rows.append(r)
            r = [0] * (d + P + 1)
            r[k] = -1
            r[-1] = hi
            rows.append(r)
        for _ in range(rng.randint(0, 3)):  # triangles / trapezoids / parametric cuts
            r = [rng.randint(-2, 2) for _ in range(d)] + [rng.randint(-1, 1) for _ in range(P)] + [rng.randint(-4, 10)]
            rows.append(r)
        stmts.append({"depth": d, "rows": rows, "box": [[lo, hi]] * d})
    refs = []
    ranks = {}
    for _ in range(rng.randint(1, 5)):
        s = rng.randrange(len(stmts))
        arr = rng.randint(0, 2)
        rk = ranks.setdefault(arr, rng.randint(1, 2))
        d = stmts[s]["depth"]
        rows = []
        for _ in range(rk):
            row = [rng.choice([-1, 0, 0, 1, 1, 2]) for _ in range(d)] + [rng.randint(-1, 1) for _ in range(P)] \
                + [rng.randint(-3, 3)]
            rows.append(row)
        refs.append({"stmt": s, "array": arr, "is_write": rng.random() < 0.35, "rank": rk, "rows": rows})
    return {"params": params, "stmts": stmts, "refs": refs}


@pytest.mark.parametrize("seed", range(40))
def test_random_blocks(seed):
    rng = random.Random(1000 + seed)
    for _ in range(25):
        blk = _rand_block(rng)
        mode = rng.choice([O.PER_ARRAY, O.COMPONENTS])
        _compare(blk, mode=mode, reuse_filter=rng.random() < 0.3, delta=rng.choice([0.3, 0.1, 0.6]),
                 compress=rng.random() < 0.5)


def test_jacobi_tile_blocks_match_kernel_closed_form():
    """Every tile of J1-like passes: the planner's bbox of `a` equals the closed form the
    Jacobi kernel stages (sp_jacobi1d_tile_footprint)."""
    for N, S, h in [(4096, 256, 16), (1000, 64, 7), (37, 8, 3), (3, 4, 1)]:
        for x0 in range(0, N, S):
            lo_i, hi_i = max(1, x0 - h + 1), min(N - 2, x0 + S + h - 2)
            rows = [[1, 0, 0], [-1, 0, h - 1], [-1, 1, -(x0 - h + 1)], [-1, -1, x0 + S - 2 + h],
                    [0, 1, -1], [0, -1, N - 2]]
            blk = {"params": [], "stmts": [{"depth": 2, "rows": rows, "box": [[0, h - 1], [0, N - 1]]}],
                   "refs": [{"stmt": 0, "array": 0, "is_write": 0, "rank": 1, "rows": [[0, 1, d]]} for d in (-1, 0, 1)]
                   + [{"stmt": 0, "array": 1, "is_write": 1, "rank": 1, "rows": [[0, 1, 0]]}]}
            p = sp.plan_buffers(blk)
            if lo_i > hi_i:
                assert p["buffers"][0]["size"] == 0
                continue
            lb, ub = sp.jacobi1d_tile_footprint(N, h, x0, S)
            assert (p["buffers"][0]["lb"], p["buffers"][0]["ub"]) == ([lb], [ub]), (N, S, h, x0)


def test_me_macroblock_block_matches_kernel_window():
    """ME tile (one MB, all valid candidates, Fig. 2 nest over (dy, dx, v, u)): the planner's
    bbox of ref equals the window the ME kernel stages (sp_me_ref_window)."""
    W, H, R = 96, 64, 8
    for by in range(H // 16):
        for bx in range(W // 16):
            x0, y0 = 16 * bx, 16 * by
            # dy in [max(-R,-y0), min(R,H-16-y0)], dx likewise, v,u in [0,15]
            dylo, dyhi = max(-R, -y0), min(R, H - 16 - y0)
            dxlo, dxhi = max(-R, -x0), min(R, W - 16 - x0)
            rows = [[1, 0, 0, 0, -dylo], [-1, 0, 0, 0, dyhi], [0, 1, 0, 0, -dxlo], [0, -1, 0, 0, dxhi],
                    [0, 0, 1, 0, 0], [0, 0, -1, 0, 15], [0, 0, 0, 1, 0], [0, 0, 0, -1, 15]]
            blk = {"params": [], "stmts": [{"depth": 4, "rows": rows}],
                   "refs": [{"stmt": 0, "array": 0, "is_write": 0, "rank": 2, "rows": [[1, 0, 1, 0, y0], [0, 1, 0, 1, x0]]},
                            {"stmt": 0, "array": 1, "is_write": 0, "rank": 2, "rows": [[0, 0, 1, 0, y0], [0, 0, 0, 1, x0]]},
                            {"stmt": 0, "array": 2, "is_write": 1, "rank": 2, "rows": [[1, 0, 0, 0, R], [0, 1, 0, 0, R]]}]}
            p = sp.plan_buffers(blk)
            (l0, l1), (u0, u1) = sp.me_ref_window(W, H, R, bx, by)
            ref = p["buffers"][0]
            assert ref["lb"] == [l0, l1] and ref["ub"] == [u0, u1]
            assert all(b["beneficial"] for b in p["buffers"])  # rank 2 < depth 4 for every ref
            assert p["buffers"][1]["lb"] == [y0, x0] and p["buffers"][1]["size"] == 256


# ---- error behaviour ------------------------------------------------------------------
def _one(rows, ref_rows, depth=1, params=()):
    return {"params": list(params), "stmts": [{"depth": depth, "rows": rows, "box": [[0, 10]] * depth}],
            "refs": [{"stmt": 0, "array": 0, "is_write": 0, "rank": len(ref_rows), "rows": ref_rows}]}


def test_unbounded_domain():
    assert sp.plan_buffers(_one([[1, 0]], [[1, 0]]))["status"] == -2


def test_empty_domain():
    p = sp.plan_buffers(_one([[1, -5], [-1, 4]], [[1, 0]]))
    assert p["status"] == 0 and p["buffers"][0]["size"] == 0 and p["buffers"][0]["ub"] == [-1]


def test_overflow():
    assert sp.plan_buffers(_one([[1, 0], [-1, 10]], [[1 << 62, 0]]))["status"] == -4


def test_smem_limit():
    blk = _one([[1, 0], [-1, 10]], [[1, 0]])
    assert sp.plan_buffers(blk, mup_elems=11)["status"] == 0
    assert sp.plan_buffers(blk, mup_elems=10)["status"] == -6


def test_enumeration_budget():
    blk = _one([[1, 0, 0], [-1, 0, 999], [0, 1, 0], [0, -1, 999]], [[1, 0, 0]], depth=2)
    assert sp.plan_buffers(blk, max_points=1000)["status"] == -5
    assert sp.plan_buffers(blk)["status"] == 0


def test_capacity_raw_abi():
    import ctypes
    blk = json.load(open(GOLD))["block"]
    # build through the binding once to get ctypes structures, then call with cap 0
    keep = []
    doms = (sp.sp_domain * 2)()
    for k, s in enumerate(blk["stmts"]):
        r = np.ascontiguousarray(np.asarray(s["rows"], dtype=np.int64))
        keep.append(r)
        doms[k] = sp.sp_domain(s["depth"], r.shape[0], r.ctypes.data_as(ctypes.POINTER(ctypes.c_int64)))
    refs = (sp.sp_ref * 5)()
    for k, rf in enumerate(blk["refs"]):
        r = np.ascontiguousarray(np.asarray(rf["rows"], dtype=np.int64))
        keep.append(r)
        refs[k] = sp.sp_ref(rf["stmt"], rf["array"], rf["is_write"], rf["rank"],
                            r.ctypes.data_as(ctypes.POINTER(ctypes.c_int64)))
    b = sp.sp_block(0, 2, 5, 0, None, doms, refs)
    n = ctypes.c_int32(0)
    st = sp.lib.sp_plan_buffers(ctypes.byref(b), None, None, 0, ctypes.byref(n), None, None)
    assert st == -3 and n.value == 2
    assert sp.lib.sp_plan_buffers(None, None, None, 0, ctypes.byref(n), None, None) == -1
    b.reserved = 1
    assert sp.lib.sp_plan_buffers(ctypes.byref(b), None, None, 0, ctypes.byref(n), None, None) == -1


@pytest.mark.parametrize("seed", range(12))
def test_random_blocks_compressed(seed):
    """§3.1.2 compression on random blocks (rank-deficient accesses are frequent: subscript
    coefficients in {-1, 0, 1, 2}): kept dimensions, sizes and F' rows equal the oracle's."""
    rng = random.Random(1000 + seed)
    dropped = 0
    for _ in range(25):
        blk = _rand_block(rng)
        for mode in (O.PER_ARRAY, O.COMPONENTS):
            o, _ = _compare(blk, mode=mode, compress=True)
            if o["status"] == 0:
                dropped += sum(b["n_dims"] < b["rank"] for b in o["buffers"])
    assert dropped > 0  # the case is exercised
