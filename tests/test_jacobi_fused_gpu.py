"""GPU parity of the persistent all-passes Jacobi (sp_jacobi1d_timetiled_fused) against the
oracle: bit-exact, like the per-pass path, on edge shapes, space tiles smaller than the halo
(dependences reaching several tiles), every time tile, J1, and J3 at full size (sampled)."""
import numpy as np
import pytest
import torch

import oracle
import paper_conf_ppopp_baskaranbkrrs08_b200 as sp
import sp_inputs

pytestmark = pytest.mark.gpu


@pytest.fixture(autouse=True)
def _persistent_at_every_time_tile(monkeypatch):
    """Below Tt = 16 sp_jacobi1d_timetiled_fused runs one launch per pass by default (faster
    when HBM binds); this module tests the persistent kernel itself at every time tile."""
    monkeypatch.setenv("SP_JACOBI_FUSED_PERSISTENT", "1")


def _run(a0, steps, tt, S=0, log=None):
    d = torch.from_numpy(a0.copy()).cuda()
    sp.jacobi1d_timetiled_fused(d, steps, tt, S, footprint_log=log)
    torch.cuda.synchronize()
    return d.cpu().numpy()


def _check(got, want):
    assert np.array_equal(got.view(np.uint32), want.view(np.uint32)), "not bit-exact"


def test_J1_config():
    a = sp_inputs.jacobi_input(4096, seed=2008)
    want = oracle.jacobi1d(a, 64)
    for S in (0, 256, 512, 16):
        _check(_run(a, 64, 16, S), want)


@pytest.mark.parametrize("n", [3, 5, 33, 64, 65, 1000, 4097])
@pytest.mark.parametrize("steps", [0, 1, 16, 17, 53, 130])
def test_edge_shapes(n, steps):
    a = sp_inputs.jacobi_input(n, seed=n * 3 + steps)
    want = oracle.jacobi1d(a, steps)
    # (16, ...) and below: the staged persistent geometry; 48 / 64: the in-place one
    for tt, S in [(16, 32), (16, 4), (5, 8), (1, 4), (16, 0), (48, 0), (64, 32), (64, 4)]:
        _check(_run(a, steps, tt, S), want)


@pytest.mark.parametrize("tt", [1, 3, 8, 16, 32, 64, 100, 128])
def test_time_tiles(tt):
    a = sp_inputs.jacobi_input(50000, seed=tt)
    want = oracle.jacobi1d(a, 333)
    _check(_run(a, 333, tt), want)
    _check(_run(a, 333, tt, 8), want)  # S << H: each tile waits on up to 2 * ceil(H / S) + 1 others


def test_footprint_log_matches_per_pass_path():
    n, steps, tt, S = 30000, 100, 16, 512
    plan = sp.jacobi1d_plan(n, steps, tt, S)
    a = sp_inputs.jacobi_input(n, seed=4)
    logs = []
    for fused in (False, True):
        log = torch.zeros(plan["passes"] * plan["tiles"] * 2, dtype=torch.int64, device="cuda")
        d = torch.from_numpy(a.copy()).cuda()
        (sp.jacobi1d_timetiled_fused if fused else sp.jacobi1d_timetiled)(d, steps, tt, S, footprint_log=log)
        torch.cuda.synchronize()
        logs.append(log.cpu().numpy())
    assert np.array_equal(logs[0], logs[1])


@pytest.mark.parametrize("tt", [64, 128])
def test_J3_size_sampled(tt):
    n, steps = 1 << 26, 1024
    a = sp_inputs.jacobi_input(n, seed=2008)
    got = _run(a, steps, tt)
    S = sp.jacobi1d_plan(n, steps, tt, 0)["persistent_space_tile"]  # the persistent launch's tiles
    rng = np.random.default_rng(7)
    idx = [0, 1, 2, n - 3, n - 2, n - 1]
    for t in [0, 1, 500, (n // S) - 1, n // S]:
        for off in (-1, 0, 1, S - 1, S + 1):
            if 0 <= t * S + off < n:
                idx.append(t * S + off)
    idx = np.unique(np.array(idx + rng.integers(0, n, 40).tolist(), dtype=np.int64))
    _check(got[idx], oracle.jacobi1d_points(a, steps, idx))


_J3_WANT = {}


@pytest.mark.parametrize("tt", [128, 64])
def test_J3_every_cell_device_and_host_paths(tt):
    """BASELINE config 3 in full: all 2^26 cells after T = 1024 steps, from the bench's
    launch (persistent, device-resident; Tt = 128 is the bench's) and from the end-to-end
    host-buffer call (wavefront order, pinned in / out), against the untiled oracle (about
    10 s of host time on 16 cores, computed once for both time tiles)."""
    n, steps = 1 << 26, 1024
    a = sp_inputs.jacobi_input(n, seed=2008)
    got = _run(a, steps, tt)
    h = torch.from_numpy(a.copy()).pin_memory()
    sp.Jacobi1DHost(n, steps, tt, 0).run(h)
    torch.cuda.synchronize()
    if "want" not in _J3_WANT:
        _J3_WANT["want"] = oracle.jacobi1d(a, steps)
    want = _J3_WANT["want"]
    _check(got, want)
    _check(h.numpy(), want)


def test_repeated_calls_reuse_flags():
    n = 100003
    a = sp_inputs.jacobi_input(n, seed=11)
    d = torch.from_numpy(a.copy()).cuda()
    w = torch.empty_like(d)
    flags = torch.full((sp.jacobi1d_plan(n, 40, 16, 0)["tiles"] + 1,), 12345, dtype=torch.int32, device="cuda")
    for _ in range(3):
        sp.jacobi1d_timetiled_fused(d, 40, 16, 0, work=w, flags=flags)
    torch.cuda.synchronize()
    _check(d.cpu().numpy(), oracle.jacobi1d(a, 120))


@pytest.mark.parametrize("tt", [1, 5, 8, 15])
def test_small_time_tiles_default_route(tt, monkeypatch):
    """Default route below Tt = 16 (per-pass launches): same bits and the same footprint log
    layout as the persistent launch."""
    monkeypatch.delenv("SP_JACOBI_FUSED_PERSISTENT", raising=False)
    n, steps = 20011, 53
    a = sp_inputs.jacobi_input(n, seed=tt)
    want = oracle.jacobi1d(a, steps)
    plan = sp.jacobi1d_plan(n, steps, tt, 0)
    logs = []
    for env in (None, "1"):
        if env:
            monkeypatch.setenv("SP_JACOBI_FUSED_PERSISTENT", env)
        log = torch.zeros(plan["passes"] * plan["persistent_tiles"] * 2, dtype=torch.int64, device="cuda")
        _check(_run(a, steps, tt, 0, log=log), want)
        logs.append(log.cpu().numpy())
    assert np.array_equal(logs[0], logs[1])
