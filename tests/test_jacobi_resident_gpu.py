"""GPU parity of the cluster-resident Jacobi (sp_jacobi1d_resident: the whole domain in one
thread-block cluster, halos exchanged every E steps through shared / distributed shared
memory; small configuration K = 12, E = 6 up to 96,768 cells, large K = 28, E = 14 above)
against the oracle, bit-exact: single warp, several warps, several CTAs of the cluster (DSMEM
exchanges), both configurations and the switch between them, the capacity limit, steps
around multiples of both exchange intervals, in place and out of place."""
import numpy as np
import pytest
import torch

import oracle
import paper_conf_ppopp_baskaranbkrrs08_b200 as sp
import sp_inputs

pytestmark = pytest.mark.gpu
SEG = 64 * 12 - 2 * 6  # owned cells per warp (small configuration, n <= 16 x 8 x SEG)
CTA = 8 * SEG
SMALL_CAP = 16 * CTA  # above it the large configuration (K = 28, E = 14) runs


def _check(got, want):
    got = got.cpu().numpy() if isinstance(got, torch.Tensor) else got
    assert np.array_equal(got.view(np.uint32), want.view(np.uint32)), "not bit-exact"


def test_capacity():
    assert sp.jacobi1d_resident_capacity() >= CTA


@pytest.mark.parametrize("n", [3, 4, 5, 33, 1000, SEG - 1, SEG, SEG + 1, 4096, CTA - 1, CTA, CTA + 1,
                               3 * CTA + 17, 8192, 32768, SMALL_CAP, SMALL_CAP + 1, 150001])
@pytest.mark.parametrize("steps", [0, 1, 5, 6, 7, 13, 14, 15, 28, 29, 64, 101])
def test_shapes(n, steps):
    a = sp_inputs.jacobi_input(n, seed=n + steps)
    d = torch.from_numpy(a.copy()).cuda()
    o = torch.empty_like(d)
    sp.jacobi1d_resident(d, steps, out=o)
    torch.cuda.synchronize()
    _check(o, oracle.jacobi1d(a, steps))
    sp.jacobi1d_resident(d, steps)  # in place
    torch.cuda.synchronize()
    _check(d, oracle.jacobi1d(a, steps))


def test_J1_and_long_run_at_capacity():
    a = sp_inputs.jacobi_input(4096, seed=2008)
    d = torch.from_numpy(a.copy()).cuda()
    sp.jacobi1d_resident(d, 64)
    torch.cuda.synchronize()
    _check(d, oracle.jacobi1d(a, 64))
    n = sp.jacobi1d_resident_capacity()
    a = sp_inputs.jacobi_input(n, seed=7)
    d = torch.from_numpy(a.copy()).cuda()
    sp.jacobi1d_resident(d, 4096)
    torch.cuda.synchronize()
    got = d.cpu().numpy()
    rng = np.random.default_rng(3)
    seg = 64 * 28 - 2 * 14
    idx = [0, 1, 2, n - 3, n - 2, n - 1] + [k * seg + o for k in (1, 7, 8, 9, 100) for o in (-1, 0, 1) if k * seg + o < n]
    idx = np.unique(np.array(idx + rng.integers(0, n, 30).tolist(), dtype=np.int64))
    _check(got[idx], oracle.jacobi1d_points(a, 4096, idx))
    with pytest.raises(sp.SPError):
        sp.jacobi1d_resident(torch.zeros(n + 1, device="cuda"), 4)


def test_prepared_call_J1():
    """jacobi1d_resident_prepared (the latency-config call form, arguments marshalled once):
    J1 out of place, called twice on the same buffers, equals the oracle."""
    a0 = sp_inputs.jacobi_input(4096, seed=2008)
    want = oracle.jacobi1d(a0, 64)
    src = torch.from_numpy(a0).cuda()
    dst = torch.empty_like(src)
    call = sp.jacobi1d_resident_prepared(src, 64, out=dst)
    call()
    call()
    torch.cuda.synchronize()
    _check(dst, want)
