"""N2: sp_tile_search (C++, §4.3 objective on Alg. 2 volumes) vs the oracle's exhaustive
evaluation (oracle/tilesearch.py on the brute-force planner), plus properties of the model."""
import pytest

import paper_conf_ppopp_baskaranbkrrs08_b200 as sp
from oracle import tilesearch as OT


def _me_like(R=4):
    # Fig. 2 nest (i, j) search positions x (k, l) pixels: SAD[i][j] += |cur[k][l] - ref[i+k][j+l]|
    return [
        {"array": 0, "is_write": 0, "rank": 2, "rows": [[1, 0, 1, 0, 0], [0, 1, 0, 1, 0]]},  # ref[i+k][j+l]
        {"array": 1, "is_write": 0, "rank": 2, "rows": [[0, 0, 1, 0, 0], [0, 0, 0, 1, 0]]},  # cur[k][l]
        {"array": 2, "is_write": 1, "rank": 2, "rows": [[1, 0, 0, 0, 0], [0, 1, 0, 0, 0]]},  # SAD[i][j] (write)
        {"array": 2, "is_write": 0, "rank": 2, "rows": [[1, 0, 0, 0, 0], [0, 1, 0, 0, 0]]},  # SAD[i][j] (read)
    ]


def _jacobi_like():
    # time-skewed (t, i) band: b[i] = f(a[i-1], a[i], a[i+1]) over a tile of (t, i)
    return [
        {"array": 0, "is_write": 0, "rank": 1, "rows": [[0, 1, -1]]},
        {"array": 0, "is_write": 0, "rank": 1, "rows": [[0, 1, 0]]},
        {"array": 0, "is_write": 0, "rank": 1, "rows": [[0, 1, 1]]},
        {"array": 1, "is_write": 1, "rank": 1, "rows": [[0, 1, 0]]},
    ]


@pytest.mark.parametrize("S,L,mup,P", [(1.0, 1.0, 0, 4), (50.0, 1.0, 300, 8), (0.1, 5.0, 200, 16), (10.0, 10.0, 120, 4)])
def test_me_like_matches_oracle(S, L, mup, P):
    ext = [16, 12, 4, 4]
    cands = [[1, 2, 4, 8, 16], [1, 3, 6, 12], [1, 2, 4], [2, 4]]
    got = sp.tile_search(ext, _me_like(), cands, mup_elems=mup, procs=P, sync_cost=S, elem_cost=L)
    want = OT.tile_search(ext, _me_like(), cands, mup_elems=mup, procs=P, sync_cost=S, elem_cost=L)
    assert got["evaluated"] == want["evaluated"]
    assert got["tile"] == want["best"]["tile"]
    assert got["cost"] == pytest.approx(want["best"]["cost"], rel=1e-12)
    assert got["local_elems"] == want["best"]["local_elems"]


def test_jacobi_like_matches_oracle():
    ext = [32, 256]
    cands = [[1, 2, 4, 8, 16, 32], [8, 16, 32, 64, 128, 256]]
    for mup in (0, 64, 200):
        got = sp.tile_search(ext, _jacobi_like(), cands, mup_elems=mup, procs=8, sync_cost=20.0, elem_cost=1.0)
        want = OT.tile_search(ext, _jacobi_like(), cands, mup_elems=mup, procs=8, sync_cost=20.0, elem_cost=1.0)
        assert got["tile"] == want["best"]["tile"] and got["cost"] == pytest.approx(want["best"]["cost"])


def test_model_properties():
    ext = [32, 256]
    cands = [[1, 2, 4, 8, 16, 32], [8, 16, 32, 64, 128, 256]]
    # a synchronisation-dominated machine prefers fewer, larger movements
    big_s = sp.tile_search(ext, _jacobi_like(), cands, procs=8, sync_cost=1e6, elem_cost=1.0)
    assert big_s["tile"][1] == 256
    # the memory limit binds: local footprint never exceeds M_up
    lim = sp.tile_search(ext, _jacobi_like(), cands, mup_elems=100, procs=8, sync_cost=1e6, elem_cost=1.0)
    assert lim["feasible"] and lim["local_elems"] <= 100
    # infeasible limit
    none = sp.tile_search(ext, _jacobi_like(), cands, mup_elems=5, procs=8)
    assert not none["feasible"]
    with pytest.raises(sp.SPError):
        sp.tile_search(ext, _jacobi_like(), [[64], [8]], procs=8)  # t > N


def test_cost_hand_derived_jacobi_band():
    """Pin of the §4.3 objective computed by hand for one tile of the Jacobi
    band (extent T = 32, N = 256; tile t = (8, 64); P = 8, S = 20, L = 1):
    array a is read (a[i-1], a[i], a[i+1]) -> one move-in per tile of the box [-1, 64]:
    V_in = 66;  array b is written (b[i]) -> one move-out per tile: V_out = 64.  Both depend
    on loop 1, so neither movement is hoisted: 4 x 4 = 16 tiles each.
    C = 16 (8*20 + 66/8) + 16 (8*20 + 64/8) = 2692 + 2688 = 5380;  local footprint 66 + 64."""
    for f in (sp.tile_search, OT.tile_search):
        r = f([32, 256], _jacobi_like(), [[8], [64]], procs=8, sync_cost=20.0, elem_cost=1.0)
        best = r if "tile" in r else r["best"]
        assert list(best["tile"]) == [8, 64]
        assert best["cost"] == pytest.approx(5380.0)
        assert best["local_elems"] == 130


def test_cost_hand_derived_matvec_hoisting():
    """Hoisting above a redundant tiling loop (reading R-T2), by hand: y[i] +=
    A[i][j] * x[j] over (i, j) with extent (64, 128), tile (16, 32), P = 4, S = 10, L = 2.
    y depends only on loop 0: moved in and out once per i-tile (4 times, 16 elements each);
    A (16 x 32) and x (32) depend on loop 1: moved in per tile (4 x 4 = 16 times).
    C = 4 (40 + 16*2/4) * 2 + 16 (40 + 512*2/4) + 16 (40 + 32*2/4) = 384 + 4736 + 896 = 6016."""
    refs = [
        {"array": 0, "is_write": 1, "rank": 1, "rows": [[1, 0, 0]]},             # y[i] (write)
        {"array": 0, "is_write": 0, "rank": 1, "rows": [[1, 0, 0]]},             # y[i] (read)
        {"array": 1, "is_write": 0, "rank": 2, "rows": [[1, 0, 0], [0, 1, 0]]},  # A[i][j]
        {"array": 2, "is_write": 0, "rank": 1, "rows": [[0, 1, 0]]},             # x[j]
    ]
    for f in (sp.tile_search, OT.tile_search):
        r = f([64, 128], refs, [[16], [32]], procs=4, sync_cost=10.0, elem_cost=2.0)
        best = r if "tile" in r else r["best"]
        assert best["cost"] == pytest.approx(6016.0)
        assert best["local_elems"] == 16 + 512 + 32
