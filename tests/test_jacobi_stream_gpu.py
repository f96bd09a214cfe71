"""GPU parity of the general persistent Jacobi (sp_jacobi1d_timetiled_stream) and of the
end-to-end host-buffer call (sp_jacobi1d_host) against the oracle, bit-exact: wavefront unit
orders (skew D), pass 0 reading / the last pass writing page-locked host memory directly,
in / out aliasing (including the single-pass case that must redirect), footprint log under
the wavefront order, and J3 at full size through the host path (light-cone samples)."""
import numpy as np
import pytest
import torch

import oracle
import paper_conf_ppopp_baskaranbkrrs08_b200 as sp
import sp_inputs

pytestmark = pytest.mark.gpu


def _check(got, want):
    got = got.cpu().numpy() if isinstance(got, torch.Tensor) else got
    assert np.array_equal(got.view(np.uint32), want.view(np.uint32)), "not bit-exact"


def _stream(a0, steps, tt, S, skew, where_in="cuda", where_out="cuda", same=False):
    t = torch.from_numpy(a0.copy())
    inp = t.cuda() if where_in == "cuda" else t.pin_memory()
    if same:
        out = inp
    else:
        out = torch.empty_like(t)
        out = out.cuda() if where_out == "cuda" else out.pin_memory()
    sp.jacobi1d_timetiled_stream(inp, out, steps, tt, S, skew)
    torch.cuda.synchronize()
    return out


@pytest.mark.parametrize("skew", [0, 2, 3, 4, 8, 256, -1])
def test_skews_J1_and_small_tiles(skew):
    a = sp_inputs.jacobi_input(4096, seed=2008)
    want = oracle.jacobi1d(a, 64)
    for tt, S in [(16, 0), (16, 256), (16, 64), (5, 8)]:
        reach = -(-sp.halo_of(tt) // (S or sp.jacobi1d_plan(4096, 64, tt, 0)["space_tile"]))
        if 0 < skew and (skew <= reach or skew & (skew - 1)):
            with pytest.raises(sp.SPError):
                _stream(a, 64, tt, S, skew)
            continue
        _check(_stream(a, 64, tt, S, skew), want)


@pytest.mark.parametrize("n", [3, 5, 65, 1000, 4097, 50001])
@pytest.mark.parametrize("steps", [0, 1, 16, 17, 40, 53])
def test_host_in_out_shapes(n, steps):
    """pinned host in and out (the last pass's move-out writes host memory), all pass counts"""
    a = sp_inputs.jacobi_input(n, seed=n + 7 * steps)
    want = oracle.jacobi1d(a, steps)
    # 16 / 5: the staged persistent geometry; 48 / 64: the in-place one (host output: its
    # staged-move-out instantiation)
    for tt, S in [(16, 0), (16, 8), (5, 4), (64, 0), (48, 8)]:
        _check(_stream(a, steps, tt, S, -1, "host", "host"), want)
        _check(_stream(a, steps, tt, S, 0, "host", "cuda"), want)
        _check(_stream(a, steps, tt, S, 16, "cuda", "host"), want)


@pytest.mark.parametrize("steps", [1, 16, 17, 32, 33, 100])
def test_in_place_aliasing(steps):
    """in == out (device and pinned host): single-pass and odd pass counts take the
    redirect + copy path, the others write the input array from the last pass"""
    a = sp_inputs.jacobi_input(20011, seed=steps)
    want = oracle.jacobi1d(a, steps)
    for where in ("cuda", "host"):
        for skew in (0, -1):
            _check(_stream(a, steps, 16, 0, skew, where, same=True), want)


@pytest.mark.parametrize("direct", [False, True])
def test_host_class_reuse_and_public_call(direct):
    """copy-engine input (chunks + ready flags) and the direct PCIe move-in; a second call on
    the same flags and buffers continues from the first one's result"""
    n, steps, tt = 300007, 200, 64
    a = sp_inputs.jacobi_input(n, seed=5)
    ctx = sp.Jacobi1DHost(n, steps, tt, direct_input=direct)
    h = torch.from_numpy(a.copy()).pin_memory()
    ctx.run(h)
    ctx.run(h)  # flags reused, state carried on: 2 * steps in total
    torch.cuda.synchronize()
    _check(h, oracle.jacobi1d(a, 2 * steps))
    _check(sp.jacobi1d(a, steps, tt), oracle.jacobi1d(a, steps))


def test_host_rejects_pageable():
    a = torch.from_numpy(sp_inputs.jacobi_input(1000, seed=1))
    ctx = sp.Jacobi1DHost(1000, 10, 16)
    with pytest.raises(sp.SPError):
        rc = sp.lib.sp_jacobi1d_host(a.data_ptr(), ctx.buf0.data_ptr(), ctx.buf1.data_ptr(), ctx.flags.data_ptr(),
                                     ctx.flags.numel(), 1000, 10, 16, 0, None)
        sp._check(rc, "sp_jacobi1d_host")


def test_footprint_log_under_wavefront_order():
    n, steps, tt, S = 30000, 100, 16, 512
    plan = sp.jacobi1d_plan(n, steps, tt, S)
    a = sp_inputs.jacobi_input(n, seed=4)
    logs = []
    for skew in (0, 2, 32):
        log = torch.zeros(plan["passes"] * plan["tiles"] * 2, dtype=torch.int64, device="cuda")
        inp = torch.from_numpy(a.copy()).cuda()
        out = torch.empty_like(inp)
        sp.jacobi1d_timetiled_stream(inp, out, steps, tt, S, skew, footprint_log=log)
        torch.cuda.synchronize()
        _check(out, oracle.jacobi1d(a, steps))
        logs.append(log.cpu().numpy())
    assert np.array_equal(logs[0], logs[1]) and np.array_equal(logs[0], logs[2])
    lg = logs[0].reshape(plan["passes"], plan["tiles"], 2)
    for p in (0, plan["passes"] - 1):
        h = min(tt, steps - p * tt)
        for t in range(plan["tiles"]):
            lb, ub = sp.jacobi1d_tile_footprint(n, h, t * S, S)
            assert (lg[p, t, 0], lg[p, t, 1]) == (lb, ub)


@pytest.mark.parametrize("tt,direct", [(64, False), (128, False), (128, True)])
def test_J3_size_host_path_sampled(tt, direct):
    """the bench's e2e call at full size: 2^26 cells, T = 1024, pinned host in/out (Tt = 128 is
    the bench's; the in-place kernel's host-output instantiation stages the last pass's
    move-out), samples around the persistent geometry's tile boundaries"""
    n, steps = 1 << 26, 1024
    a = sp_inputs.jacobi_input(n, seed=2008)
    h = torch.from_numpy(a.copy()).pin_memory()
    sp.Jacobi1DHost(n, steps, tt, direct_input=direct).run(h)
    torch.cuda.synchronize()
    got = h.numpy()
    S = sp.jacobi1d_plan(n, steps, tt, 0)["persistent_space_tile"]
    rng = np.random.default_rng(11)
    idx = [0, 1, 2, n - 3, n - 2, n - 1]
    for t in [0, 1, 255, 256, 257, 5000, (n // S) - 1, n // S]:
        for off in (-1, 0, 1, S - 1):
            if 0 <= t * S + off < n:
                idx.append(t * S + off)
    idx = np.unique(np.array(idx + rng.integers(0, n, 40).tolist(), dtype=np.int64))
    _check(got[idx], oracle.jacobi1d_points(a, steps, idx))


@pytest.mark.parametrize("n", [3, 4099, (1 << 21) - 5, (1 << 21) + 7, 3 * (1 << 21) + 1000])
@pytest.mark.parametrize("tt", [48, 64, 128])
def test_host_copy_engine_chunks(n, tt):
    """copy-engine input across chunk boundaries (SP_JACOBI_HOST_CHUNK = 2^21 cells): one
    chunk, a chunk plus a few cells, several chunks; every cell equals the oracle"""
    steps = 2 * tt + 5
    a = sp_inputs.jacobi_input(n, seed=n % 97 + tt)
    h = torch.from_numpy(a.copy()).pin_memory()
    ctx = sp.Jacobi1DHost(n, steps, tt)
    assert ctx.flags.numel() > sp.jacobi1d_plan(n, steps, tt, 0)["persistent_tiles"] + 1
    ctx.run(h)
    torch.cuda.synchronize()
    _check(h, oracle.jacobi1d(a, steps))


def test_host_paths_under_launch_blocking():
    """The host-buffer calls stay correct when every launch is serialised
    (CUDA_LAUNCH_BLOCKING=1, as under ncu): their kernels spin on ready flags set by copies on a
    side stream, so those copies must be enqueued before the launch (a launch-first order
    deadlocked until the kernel's trap)."""
    import os
    import subprocess
    import sys
    code = r"""
import numpy as np, torch, oracle, sp_inputs
import paper_conf_ppopp_baskaranbkrrs08_b200 as sp
n, steps = 300007, 150
a = sp_inputs.jacobi_input(n, seed=9)
h = torch.from_numpy(a.copy()).pin_memory()
sp.Jacobi1DHost(n, steps, 64).run(h)
torch.cuda.synchronize()
assert np.array_equal(h.numpy().view(np.uint32), oracle.jacobi1d(a, steps).view(np.uint32))
W, H, R = 352, 288, 16
fr = sp_inputs.me_sequence(4, W, H, R, seed=3)
mv, sad = sp.me_search(fr, W, H, R)
for p in range(3):
    omv, osad, _ = oracle.me_search(fr[p], fr[p + 1], W, H, R)
    assert np.array_equal(mv[p].numpy().reshape(-1, 2), omv)
    assert np.array_equal(sad[p].numpy().view(np.uint32).reshape(-1), osad)
print("ok")
"""
    env = dict(os.environ, CUDA_LAUNCH_BLOCKING="1")
    root = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
    r = subprocess.run([sys.executable, "-c", code], cwd=root, env=env, capture_output=True, text=True, timeout=300)
    assert r.returncode == 0 and r.stdout.strip().endswith("ok"), r.stderr[-2000:]
