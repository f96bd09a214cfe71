"""Pins for the planner oracle (oracle/planner.py) — what the paper and the mathematics fix.

* Figure 1's printed plan (tests/golden/figure1.json): bounds, offsets,
  declared extents, local access functions, and the exact move-in / move-out sets the
  printed loop nests scan.
* Hand-derived facts about Figure 1's data spaces (COMPONENTS partition, V_in / V_out,
  Alg. 1 outcome), derived in the comments below from the loop bounds, not from the
  oracle.
* 1-D toys for Algorithm 1 whose outcome follows from counting by hand.
"""
import json
import os

import numpy as np

from oracle import planner as P

GOLD = os.path.join(os.path.dirname(__file__), "golden", "figure1.json")


def _fig1():
    with open(GOLD) as f:
        return json.load(f)


def _scan(loops):
    """Enumerate the cells a printed loop nest visits."""
    cells = set()
    for nest in loops:
        for i in range(nest["i"][0], nest["i"][1] + 1):
            lo = eval(nest["j"][0], {"max": max, "min": min}, {"i": i})  # printed bound expression
            hi = eval(nest["j"][1], {"max": max, "min": min}, {"i": i})
            for j in range(lo, hi + 1):
                cells.add((i, j))
    return cells


def _set_of(plan_block, ref_ids, want_write):
    blk = plan_block
    out = set()
    for k in ref_ids:
        r = blk["refs"][k]
        if bool(r["is_write"]) != want_write:
            continue
        st = blk["stmts"][r["stmt"]]
        pts = P.enumerate_domain(st, blk["params"], st["box"])
        out |= P._as_set(P.data_space(r, pts, blk["params"]))
    return out


def test_figure1_printed_bounds_and_extents():
    g = _fig1()
    plan = P.plan_buffers(g["block"], mode=P.PER_ARRAY)
    assert plan["status"] == P.OK
    bufs = plan["buffers"]
    assert [b["array"] for b in bufs] == [0, 1]
    for b, name in zip(bufs, ["A", "B"]):
        pr = g["printed"][name]
        assert b["lb"] == pr["lb"], name
        assert b["ub"] == pr["ub"], name
        assert b["lb"] == pr["offset"], name  # g = (lb_1..lb_n)
        assert [u - l + 1 for l, u in zip(b["lb"], b["ub"])] == pr["decl"], name
        assert b["size"] == pr["decl"][0] * pr["decl"][1]


def test_figure1_printed_local_access_functions():
    g = _fig1()
    plan = P.plan_buffers(g["block"], mode=P.PER_ARRAY)
    for la in g["printed"]["local_access"]:
        assert plan["local_rows"][la["ref"]] == la["rows"], la["text"]
    assert plan["ref_buf"] == [0, 0, 1, 0, 1]


def test_figure1_printed_move_sets():
    g = _fig1()
    plan = P.plan_buffers(g["block"], mode=P.PER_ARRAY)
    blk = g["block"]
    for b, name in zip(plan["buffers"], ["A", "B"]):
        pr = g["printed"][name]
        mi = _scan(pr["move_in_loops"])
        mo = _scan(pr["move_out_loops"])
        # the printed loops scan exactly the union of read (write) data spaces
        assert _set_of(blk, b["refs"], False) == mi, name
        assert _set_of(blk, b["refs"], True) == mo, name
        assert b["in_count"] == len(mi) and b["out_count"] == len(mo)
        arr = np.array(sorted(mi))
        assert b["in_lb"] == arr.min(0).tolist() and b["in_ub"] == arr.max(0).tolist()
        arr = np.array(sorted(mo))
        assert b["out_lb"] == arr.min(0).tolist() and b["out_ub"] == arr.max(0).tolist()
    # printed counts: A move-in = 5*10 + sum_{i=20..28} (min(15,i-9) - max(i-13,11) + 1) = 50 + 25
    assert plan["buffers"][0]["in_count"] == 75
    assert plan["buffers"][0]["out_count"] == 25
    assert plan["buffers"][1]["in_count"] == 90
    assert plan["buffers"][1]["out_count"] == 70


def test_figure1_components_hand_derived():
    # Data spaces of A (from the loop bounds i,j in [10,14], k in [11,20]):
    #   W1 = A[i][j+1]   = {10..14} x {11..15}                     (25 cells)
    #   R1 = A[i+j][j+1] = {(i+j, j+1)}: rows 20..28, cols 11..15   (25 cells, injective map)
    #   R2 = A[i][k]     = {10..14} x {11..20}                     (50 cells)
    # W1 ⊂ R2, R1 is disjoint from both  ⇒ components {W1,R2} (bbox 10..14 x 11..20, 50)
    # and {R1} (bbox 20..28 x 11..15, 45).
    # B: W = B[i][j+k] = {10..14} x {21..34} (70); R = B[i+j][k] = {20..28} x {11..20} (90);
    #   disjoint ⇒ two components.
    g = _fig1()
    plan = P.plan_buffers(g["block"], mode=P.COMPONENTS)
    got = [(b["array"], b["lb"], b["ub"], b["size"]) for b in plan["buffers"]]
    assert got == [
        (0, [10, 11], [14, 20], 50),
        (0, [20, 11], [28, 15], 45),
        (1, [10, 21], [14, 34], 70),
        (1, [20, 11], [28, 20], 90),
    ]


def test_figure1_volumes_and_reuse_hand_derived():
    # V_in(A): read spaces R1, R2 are disjoint components: 45 + 50 = 95; V_out(A) = |W1 bbox| = 25.
    # V_in(B) = 90 (one read space), V_out(B) = 70.
    # Alg. 1: A[i][k] in the 3-deep S2 has rank 2 < 3 ⇒ A beneficial (non-constant reuse);
    # B[i][j+k] in S2 has rank 2 < 3 ⇒ B beneficial.  Pairwise overlaps: A: |W1∩R2| = 25,
    # the other pairs are empty; B: 0.
    g = _fig1()
    plan = P.plan_buffers(g["block"], mode=P.PER_ARRAY)
    A, B = plan["buffers"]
    assert (A["v_in_ub"], A["v_out_ub"], B["v_in_ub"], B["v_out_ub"]) == (95, 25, 90, 70)
    assert A["beneficial"] == 1 and B["beneficial"] == 1
    assert A["overlap"] == 25 and B["overlap"] == 0


def _toy(rows_list, depth=1, lo=0, hi=9):
    stmts = [{"depth": depth, "rows": [[1] + [0] * (depth - 1) + [-lo], [-1] + [0] * (depth - 1) + [hi]]
              + [[0] * d + [1] + [0] * (depth - d - 1) + [0] for d in range(1, depth)]
              + [[0] * d + [-1] + [0] * (depth - d - 1) + [hi] for d in range(1, depth)],
              "box": [[lo, hi]] * depth}]
    refs = [{"stmt": 0, "array": 0, "is_write": 0, "rank": 1, "rows": [r]} for r in rows_list]
    return {"params": [], "stmts": stmts, "refs": refs}


def test_alg1_toys():
    # i in [0,9], A[i] & A[i+1]: overlap {1..9} = 9 cells, union {0..10} = 11; 9 > 0.3*11 ⇒ yes.
    p = P.plan_buffers(_toy([[1, 0], [1, 1]]))
    b = p["buffers"][0]
    assert (b["overlap"], b["union_count"], b["beneficial"]) == (9, 11, 1)
    # A[i] & A[i+10]: disjoint ⇒ 0 ⇒ no (full rank: no non-constant reuse).
    b = P.plan_buffers(_toy([[1, 0], [1, 10]]))["buffers"][0]
    assert (b["overlap"], b["beneficial"]) == (0, 0)
    # A[2i] & A[2i+1]: evens vs odds ⇒ disjoint ⇒ no; bbox [0,19] size 20 although 20 cells used.
    b = P.plan_buffers(_toy([[2, 0], [2, 1]]))["buffers"][0]
    assert (b["overlap"], b["beneficial"], b["lb"], b["ub"], b["size"]) == (0, 0, [0], [19], 20)
    # exactly at the threshold is NOT beneficial (strict >): A[i] & A[i+7] over [0,9]:
    # overlap {7..9} = 3, union {0..16} = 17, 0.3*17 = 5.1 ⇒ no.
    b = P.plan_buffers(_toy([[1, 0], [1, 7]]))["buffers"][0]
    assert (b["overlap"], b["union_count"], b["beneficial"]) == (3, 17, 0)
    # rank test: A[i] inside a 2-deep nest (i, j): rank 1 < 2 ⇒ yes regardless of overlap.
    b = P.plan_buffers(_toy([[1, 0, 0]], depth=2))["buffers"][0]
    assert b["beneficial"] == 1


def test_reuse_filter_drops_nonbeneficial():
    p = P.plan_buffers(_toy([[1, 0], [1, 10]]), reuse_filter=True)
    assert p["buffers"] == [] and p["ref_buf"] == [-1, -1]
    # unstaged refs keep their global access functions
    assert p["local_rows"] == [[[1, 0]], [[1, 10]]]


def test_empty_domain_gives_size_zero_buffer():
    blk = {"params": [], "stmts": [{"depth": 1, "rows": [[1, -5], [-1, 4]], "box": [[0, 9]]}],
           "refs": [{"stmt": 0, "array": 3, "is_write": 0, "rank": 1, "rows": [[1, 0]]}]}
    b = P.plan_buffers(blk)["buffers"][0]
    assert (b["size"], b["lb"], b["ub"], b["in_count"]) == (0, [0], [-1], 0)


def test_exact_rank():
    assert P.exact_rank([[1, 2], [2, 4]]) == 1
    assert P.exact_rank([[1, 1, 0], [0, 1, 1], [1, 0, -1]]) == 2
    assert P.exact_rank([[0, 0]]) == 0
    assert P.exact_rank([[3, 0], [0, 5]]) == 2


def test_jacobi_tile_footprint_closed_form():
    """H3 closed forms: a tile (x0, h) of width S over N cells reads
    a[max(0,x0-h) .. min(N-1,x0+S-1+h)] — derived here by hand from the overlapped tile's
    iteration space t in [0,h), i in [x0-h+1+t, x0+S-2+h-t] ∩ [1, N-2] with refs a[i-1],
    a[i], a[i+1] — and writes b over [max(1,x0-h+1), min(N-2,x0+S+h-2)]."""
    for N, S, h in [(10, 4, 2), (64, 16, 5), (100, 16, 16), (3, 1, 1), (37, 7, 3)]:
        for x0 in range(0, N, S):
            lo_i, hi_i = max(1, x0 - h + 1), min(N - 2, x0 + S + h - 2)
            if lo_i > hi_i:
                continue
            # statement over (t, i): 0<=t<=h-1, i >= x0-h+1+t, i <= x0+S-2+h-t, 1<=i<=N-2
            rows = [[1, 0, 0], [-1, 0, h - 1], [-1, 1, -(x0 - h + 1)], [-1, -1, x0 + S - 2 + h],
                    [0, 1, -1], [0, -1, N - 2]]
            blk = {"params": [], "stmts": [{"depth": 2, "rows": rows, "box": [[0, h - 1], [0, N - 1]]}],
                   "refs": [{"stmt": 0, "array": 0, "is_write": 0, "rank": 1, "rows": [[0, 1, d]]} for d in (-1, 0, 1)]
                   + [{"stmt": 0, "array": 1, "is_write": 1, "rank": 1, "rows": [[0, 1, 0]]}]}
            p = P.plan_buffers(blk)
            a, b = p["buffers"]
            # the trapezoid is non-empty at t=0 here, so these are the closed forms
            assert a["lb"] == [max(0, x0 - h)] and a["ub"] == [min(N - 1, x0 + S - 1 + h)], (N, S, h, x0)
            assert b["lb"] == [lo_i] and b["ub"] == [hi_i]
            assert a["beneficial"] == 1  # rank([0,1]) = 1 < depth 2


# ---- §3.1.2 dimension compression (reading R-P8), hand-derived -------------
def _block1(ref_rows, lo=0, hi=9, rank=2, depth=1, extra_refs=()):
    """One statement over i in [lo, hi] (or (i, j) in [lo, hi]^2 for depth 2), one read ref
    (plus extra_refs) of array 0."""
    rows = []
    for k in range(depth):
        r = [0] * (depth + 1)
        r[k], r[-1] = 1, -lo
        rows.append(r)
        r = [0] * (depth + 1)
        r[k], r[-1] = -1, hi
        rows.append(r)
    refs = [{"stmt": 0, "array": 0, "is_write": 0, "rank": rank, "rows": ref_rows}]
    refs += [{"stmt": 0, "array": 0, "is_write": 0, "rank": rank, "rows": rr} for rr in extra_refs]
    return {"params": [], "stmts": [{"depth": depth, "rows": rows, "box": [[lo, hi]] * depth}], "refs": refs}


def test_compress_diagonal():
    # A[i][i], i = 0..9: the data space is a segment of the diagonal; the second subscript
    # equals the first, so the local array is 1-D with 10 elements instead of the 10 x 10 box
    b = P.plan_buffers(_block1([[1, 0], [1, 0]]), compress=True)
    buf = b["buffers"][0]
    assert buf["kept"] == [0] and buf["n_dims"] == 1 and buf["size"] == 10
    assert buf["lb"] == [0, 0] and buf["ub"] == [9, 9]  # the bounding box is still reported
    assert b["local_rows"][0] == [[1, 0], [0, 0]]  # F' = first row only; g = (0, ...)
    assert P.plan_buffers(_block1([[1, 0], [1, 0]]))["buffers"][0]["size"] == 100  # R-P5 default


def test_compress_affine_second_subscript_and_holes():
    # A[i][2i + 1]: second subscript an affine function of the first -> 1-D, 10 elements
    buf = P.plan_buffers(_block1([[1, 0], [2, 1]]), compress=True)["buffers"][0]
    assert buf["kept"] == [0] and buf["size"] == 10
    # A[2i][i]: the first subscript runs over 0, 2, ..., 18 and determines the second: kept
    # dimension 0 with bounds [0, 18] -> 19 elements (the paper's size is the hull's extent,
    # holes included)
    buf = P.plan_buffers(_block1([[2, 0], [1, 0]]), compress=True)["buffers"][0]
    assert buf["kept"] == [0] and buf["lb"] == [0, 0] and buf["ub"] == [18, 9] and buf["size"] == 19


def test_compress_plane_in_3d_and_constant_dimension():
    # A[i][j][i + j], 0 <= i, j <= 3: a 2-D plane in 3-D; the third subscript is dropped:
    # 4 x 4 = 16 elements instead of 4 x 4 x 7
    blk = _block1([[1, 0, 0], [0, 1, 0], [1, 1, 0]], lo=0, hi=3, rank=3, depth=2)
    buf = P.plan_buffers(blk, compress=True)["buffers"][0]
    assert buf["kept"] == [0, 1] and buf["n_dims"] == 2 and buf["size"] == 16
    assert P.plan_buffers(blk)["buffers"][0]["size"] == 4 * 4 * 7
    # A[5][i]: the constant first subscript is dropped (it is an affine function of no
    # dimension); the size is the same as the box's (extent 1): 10
    buf = P.plan_buffers(_block1([[0, 5], [1, 0]]), compress=True)["buffers"][0]
    assert buf["kept"] == [1] and buf["size"] == 10


def test_compress_union_of_two_lines_is_not_compressed():
    # A[i][i] and A[i][i + 1]: two parallel segments; their affine hull is the plane, so
    # both dimensions stay: box [0, 9] x [0, 10] = 110 elements
    blk = _block1([[1, 0], [1, 0]], extra_refs=[[[1, 0], [1, 1]]])
    buf = P.plan_buffers(blk, compress=True)["buffers"][0]
    assert buf["kept"] == [0, 1] and buf["size"] == 110


def test_compress_single_point_and_dimension_order():
    # A[3][4] for every i: one point, a 0-dimensional hull -> size 1 (empty product)
    buf = P.plan_buffers(_block1([[0, 3], [0, 4]]), compress=True)["buffers"][0]
    assert buf["kept"] == [] and buf["n_dims"] == 0 and buf["size"] == 1
    # A[i][9 - i]: dimensions are kept in global order, so the FIRST one stays (CLooG scans
    # the hull's dimensions in order and expresses the later one through it)
    buf = P.plan_buffers(_block1([[1, 0], [-1, 9]]), compress=True)["buffers"][0]
    assert buf["kept"] == [0] and buf["size"] == 10
