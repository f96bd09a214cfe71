"""GPU parity of the time-tiled Jacobi path (libsp sp_jacobi1d_timetiled and friends)
against the CPU oracle (oracle.jacobi1d) on the same seeded inputs.

Bar (north_star): max relative error <= 1e-5; the kernel performs the identical fp32
operation sequence (no contraction), so the tests demand bit equality, which implies it."""
import numpy as np
import pytest
import torch

import oracle
import paper_conf_ppopp_baskaranbkrrs08_b200 as sp
import sp_inputs

pytestmark = pytest.mark.gpu

REL_TOL = 1e-5


def _run(a0, steps, tt, S=0):
    d = torch.from_numpy(a0.copy()).cuda()
    sp.jacobi1d_timetiled(d, steps, tt, S)
    torch.cuda.synchronize()
    return d.cpu().numpy()


def _check(got, want):
    rel = np.max(np.abs(got.astype(np.float64) - want.astype(np.float64)) / np.abs(want.astype(np.float64)))
    assert rel <= REL_TOL, rel
    assert np.array_equal(got.view(np.uint32), want.view(np.uint32)), "not bit-exact"


def test_J1_config():
    # BASELINE config 1: N = 4096, T = 64, time tile 16
    a = sp_inputs.jacobi_input(4096, seed=2008)
    want = oracle.jacobi1d(a, 64)
    _check(_run(a, 64, 16), want)
    _check(_run(a, 64, 16, 256), want)
    _check(_run(a, 64, 16, 512), want)


@pytest.mark.parametrize("n", [3, 4, 5, 7, 31, 32, 33, 63, 64, 65, 131, 1000, 4097])
@pytest.mark.parametrize("steps", [0, 1, 15, 16, 17, 53])
def test_edge_shapes(n, steps):
    a = sp_inputs.jacobi_input(n, seed=n * 7 + steps)
    want = oracle.jacobi1d(a, steps)
    for tt, S in [(16, 32), (16, 0), (5, 8), (1, 4)]:
        _check(_run(a, steps, tt, S), want)


@pytest.mark.parametrize("tt", [1, 2, 3, 4, 8, 12, 16, 24, 32, 64, 128])
def test_time_tiles(tt):
    a = sp_inputs.jacobi_input(20000, seed=tt)
    want = oracle.jacobi1d(a, 70)
    _check(_run(a, 70, tt), want)
    S = sp.jacobi1d_plan(20000, 70, tt, 0)["space_tile"]
    _check(_run(a, 70, tt, max(4, (S // 3) & ~3)), want)


@pytest.mark.parametrize("n,steps,tt,S", [(4099, 37, 16, 256), (4099, 3, 1, 4), (100003, 96, 32, 0), (5, 3, 1, 4)])
def test_every_cell_written_by_tma_stores(n, steps, tt, S):
    """Odd pass count: the result is copied back from the work buffer, which the kernel
    writes only through TMA bulk stores (+ the ragged tail).  Poison work with NaN first;
    a cell the pass failed to write would surface as NaN (compute-sanitizer's initcheck
    does not track bulk-async stores, so this test is the evidence it cannot give)."""
    a0 = sp_inputs.jacobi_input(n, seed=n + steps)
    d = torch.from_numpy(a0.copy()).cuda()
    w = torch.full_like(d, float("nan"))
    sp.jacobi1d_timetiled(d, steps, tt, S, work=w)
    torch.cuda.synchronize()
    assert -(-steps // tt) % 2 == 1
    _check(d.cpu().numpy(), oracle.jacobi1d(a0, steps))


def test_fixed_points_on_gpu():
    r = sp_inputs.jacobi_ramp(100000)
    assert np.array_equal(_run(r, 64, 16), r)
    o = sp_inputs.jacobi_ones(9999)
    assert np.array_equal(_run(o, 33, 16), o)


def test_footprint_log_equals_planner_closed_form():
    n, steps, tt, S = 5000, 37, 16, 256
    plan = sp.jacobi1d_plan(n, steps, tt, S)
    log = torch.full((plan["passes"], plan["tiles"], 2), -7, dtype=torch.int64, device="cuda")
    d = torch.from_numpy(sp_inputs.jacobi_input(n, seed=4)).cuda()
    sp.jacobi1d_timetiled(d, steps, tt, S, footprint_log=log)
    torch.cuda.synchronize()
    log = log.cpu().numpy()
    for p in range(plan["passes"]):
        h = min(tt, steps - p * tt)
        for t in range(plan["tiles"]):
            x0 = t * S
            assert tuple(log[p, t]) == sp.jacobi1d_tile_footprint(n, h, x0, S)
            assert log[p, t, 0] == max(0, x0 - h) and log[p, t, 1] == min(n - 1, x0 + S - 1 + h)
    # and the planner derives the same boxes from the tile's iteration space (sample)
    for x0, h in [(0, 16), (2560, 16), (4864, 5)]:
        rows = [[1, 0, 0], [-1, 0, h - 1], [-1, 1, -(x0 - h + 1)], [-1, -1, x0 + S - 2 + h], [0, 1, -1], [0, -1, n - 2]]
        blk = {"params": [], "stmts": [{"depth": 2, "rows": rows}],
               "refs": [{"stmt": 0, "array": 0, "is_write": 0, "rank": 1, "rows": [[0, 1, d]]} for d in (-1, 0, 1)]}
        b = sp.plan_buffers(blk)["buffers"][0]
        p = [pp for pp in range(plan["passes"]) if min(tt, steps - pp * tt) == h][0]
        assert (b["lb"][0], b["ub"][0]) == tuple(log[p, x0 // S])


def test_J3_size_sampled():
    """BASELINE config 3 (N = 2^26, T = 1024) in the bench launch configuration; parity on
    sampled cells (tile and warp-strip edges + random) by light-cone windows."""
    n, steps, tt = 1 << 26, 1024, 16
    a = sp_inputs.jacobi_input(n, seed=2008)
    got = _run(a, steps, tt)
    S = sp.jacobi1d_plan(n, steps, tt, 0)["space_tile"]
    rng = np.random.default_rng(0)
    idx = [0, 1, 2, n - 3, n - 2, n - 1]
    for t in [0, 1, 7, 1000, (n // S) - 1, n // S]:
        for off in (-1, 0, 1, S // 2, S - 1, S + 1):
            i = t * S + off
            if 0 <= i < n:
                idx.append(i)
    idx += rng.integers(0, n, 40).tolist()
    idx = np.unique(np.array(idx, dtype=np.int64))
    want = oracle.jacobi1d_points(a, steps, idx)
    _check(got[idx], want)


def test_J5_full_size_sampled():
    """BASELINE config 5 at its full size on one GPU: N = 2^30, T = 4096, Tt = 16 (8 GiB of
    a + work), first as one domain, then through the multi-GPU pass loop with the P = 8 slab
    decomposition (loopback transport: the same slabs, halos and segment kernel the 8-GPU
    run uses).  Parity on sampled cells by light-cone windows of width 2T + 1 = 8193
    (SURVEY §8(d) J5): every slab boundary +- {0, 1, Tt - 1, Tt, Tt + 1}, the domain edges,
    and 64 random cells."""
    from paper_conf_ppopp_baskaranbkrrs08_b200.partition import jacobi_slabs
    n, steps, tt, P = 1 << 30, 4096, 16, 8
    H = sp.halo_of(tt)
    a = sp_inputs.jacobi_input(n, seed=2008)
    slabs = jacobi_slabs(n, P, H)
    idx = [0, 1, 2, n - 3, n - 2, n - 1]
    for xb, _ in slabs[1:]:
        for off in (0, 1, tt - 1, tt, tt + 1):
            idx += [xb - off, xb + off]
    idx += np.random.default_rng(5).integers(0, n, 64).tolist()
    idx = np.unique(np.array(idx, dtype=np.int64))
    want = oracle.jacobi1d_points(a, steps, idx)
    d0 = torch.from_numpy(a).cuda()
    del a
    tidx = torch.from_numpy(idx).cuda()
    d = d0.clone()
    sp.jacobi1d_timetiled(d, steps, tt)
    torch.cuda.synchronize()
    _check(d[tidx].cpu().numpy(), want)
    del d
    locs, works = [], []
    for xb, nl in slabs:
        buf = torch.zeros(nl + 2 * H, dtype=torch.float32, device="cuda")
        lo, hi = max(0, xb - H), min(n, xb + nl + H)
        buf[lo - (xb - H): hi - (xb - H)] = d0[lo:hi]
        locs.append(buf)
        works.append(torch.zeros_like(buf))
    del d0
    sp.jacobi1d_timetiled_loopback(locs, works, n, [s[0] for s in slabs], [s[1] for s in slabs], steps, tt)
    torch.cuda.synchronize()
    got = []
    for i in idx.tolist():
        r = max(k for k in range(P) if slabs[k][0] <= i)
        got.append(locs[r][H + i - slabs[r][0]].item())
    _check(np.array(got, dtype=np.float32), want)


@pytest.mark.parametrize("P", [2, 3, 4])
def test_loopback_partition_equals_oracle(P):
    """The multi-GPU pass loop (slabs + halo exchange + segment kernel) with the
    single-GPU loopback transport."""
    from paper_conf_ppopp_baskaranbkrrs08_b200.partition import jacobi_slabs
    n, steps, tt = 30011, 45, 16
    H = sp.halo_of(tt)
    a = sp_inputs.jacobi_input(n, seed=P)
    want = oracle.jacobi1d(a, steps)
    slabs = jacobi_slabs(n, P, H)
    locs, works = [], []
    for xb, nl in slabs:
        buf = torch.zeros(nl + 2 * H, dtype=torch.float32, device="cuda")
        lo, hi = max(0, xb - H), min(n, xb + nl + H)
        buf[lo - (xb - H): hi - (xb - H)] = torch.from_numpy(a[lo:hi]).cuda()
        locs.append(buf)
        works.append(torch.zeros_like(buf))
    sp.jacobi1d_timetiled_loopback(locs, works, n, [s[0] for s in slabs], [s[1] for s in slabs], steps, tt, 256)
    torch.cuda.synchronize()
    got = np.concatenate([locs[r][H:H + slabs[r][1]].cpu().numpy() for r in range(P)])
    _check(got, want)


@pytest.mark.parametrize("bounds,steps,tt", [([0, 40, 200, 240, 401], 45, 16), ([0, 36, 72, 108, 150], 40, 16),
                                             ([0, 12, 400, 1000], 23, 5), ([0, 1000, 1004 + 3000], 70, 32)])
def test_loopback_split_schedule_mixed_slabs(bounds, steps, tt):
    """The overlapped schedule (edge segments, halo exchange on a side stream, interior
    segments) with slabs shorter and longer than 3H side by side (short ones run whole)."""
    n = bounds[-1]
    H = sp.halo_of(tt)
    a = sp_inputs.jacobi_input(n, seed=n + steps)
    want = oracle.jacobi1d(a, steps)
    slabs = [(b, e - b) for b, e in zip(bounds[:-1], bounds[1:])]
    assert all(nl >= H for _, nl in slabs) and all(xb % 4 == 0 for xb, _ in slabs)
    locs, works = [], []
    for xb, nl in slabs:
        buf = torch.zeros(nl + 2 * H, dtype=torch.float32, device="cuda")
        lo, hi = max(0, xb - H), min(n, xb + nl + H)
        buf[lo - (xb - H): hi - (xb - H)] = torch.from_numpy(a[lo:hi]).cuda()
        locs.append(buf)
        works.append(torch.zeros_like(buf))
    sp.jacobi1d_timetiled_loopback(locs, works, n, [s[0] for s in slabs], [s[1] for s in slabs], steps, tt, 8)
    torch.cuda.synchronize()
    got = np.concatenate([locs[r][H:H + slabs[r][1]].cpu().numpy() for r in range(len(slabs))])
    _check(got, want)


def test_pass_segment_rejects_missing_halo():
    src = torch.zeros(1000, device="cuda")
    dst = torch.zeros(1000, device="cuda")
    with pytest.raises(sp.SPError):
        sp.jacobi1d_pass_segment(src, dst, 5000, 100, 104, 900, 16, 16)  # needs g0 <= 104-16


def test_host_api_end_to_end():
    a = sp_inputs.jacobi_input(100003, seed=9)
    got = sp.jacobi1d(a, 40, 16).numpy()
    _check(got, oracle.jacobi1d(a, 40))


def test_dist_path_single_rank_nccl():
    """The NCCL layer of the multi-GPU path (dlopen, unique id, communicator, distributed pass
    loop) on the one GPU this box has: a single rank owning the whole domain."""
    n, steps, tt = 20011, 70, 16
    H = sp.halo_of(tt)
    a = sp_inputs.jacobi_input(n, seed=21)
    comm = sp.Comm(sp.get_unique_id(), 1, 0, torch.cuda.current_device())
    try:
        buf = torch.zeros(n + 2 * H, dtype=torch.float32, device="cuda")
        buf[H:H + n] = torch.from_numpy(a).cuda()
        work = torch.zeros_like(buf)
        comm.jacobi1d_timetiled_dist(buf, work, n, 0, n, steps, tt)
        torch.cuda.synchronize()
        _check(buf[H:H + n].cpu().numpy(), oracle.jacobi1d(a, steps))
        # all-gather of one rank is a copy
        src = torch.arange(100, dtype=torch.int32, device="cuda")
        dst = torch.zeros_like(src)
        comm.allgather(src, dst)
        torch.cuda.synchronize()
        assert torch.equal(src, dst)
        assert comm.async_error() == 0  # failure detection: a healthy communicator
    finally:
        comm.destroy()
