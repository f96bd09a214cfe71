"""One process driving several GPUs (cudaSetDevice between calls): the library's per-device
launch state (ME grid caps and shared-memory attributes, ME counters, tensor-map cache,
Jacobi occupancy cache, the library-owned copy stream) must be set up on each device and
never leak across devices.  Alternates devices call by call and checks every result against
the oracle.  Skips when the box has one GPU (the driver's GPU tier has one); the one-device
variant still selects the device explicitly before every call."""
import numpy as np
import pytest
import torch

import oracle
import paper_conf_ppopp_baskaranbkrrs08_b200 as sp
import sp_inputs

pytestmark = pytest.mark.gpu


def _round(dev, fr, W, H, R, a0, steps):
    torch.cuda.set_device(dev)
    d = torch.device("cuda", dev)
    mv, sad, _ = sp.me_search_sequence(torch.from_numpy(fr).to(d), W, H, R)
    a = torch.from_numpy(a0.copy()).to(d)
    sp.jacobi1d_timetiled_fused(a, steps, 16, 0)
    mvh, sadh = sp.MESearchHost(fr.shape[0], W, H, fr.shape[2], R, device=d).run(torch.from_numpy(fr).pin_memory())
    torch.cuda.synchronize(d)
    return mv.cpu().numpy(), sad.cpu().numpy().view(np.uint32), a.cpu().numpy(), mvh.numpy(), sadh.numpy()


def _check_all(devs):
    W, H, R = 352, 288, 16
    fr = sp_inputs.me_sequence(3, W, H, R, seed=17)
    omv = [oracle.me_search(fr[p], fr[p + 1], W, H, R)[:2] for p in range(2)]
    a0 = sp_inputs.jacobi_input(50_001, seed=8)
    want = oracle.jacobi1d(a0, 40)
    for dev in devs:
        mv, sad, a, mvh, sadh = _round(dev, fr, W, H, R, a0, 40)
        for p in range(2):
            assert np.array_equal(mv[p].reshape(-1, 2), omv[p][0]), dev
            assert np.array_equal(sad[p].reshape(-1), omv[p][1]), dev
            assert np.array_equal(mvh[p].reshape(-1, 2), omv[p][0]), dev
            assert np.array_equal(sadh[p].reshape(-1).view(np.uint32), omv[p][1]), dev
        assert np.array_equal(a.view(np.uint32), want.view(np.uint32)), dev


def test_one_device_selected_explicitly():
    _check_all([0, 0])


@pytest.mark.skipif(torch.cuda.device_count() < 2, reason="needs two GPUs in one process")
def test_alternating_devices_in_one_process():
    n = torch.cuda.device_count()
    _check_all([0, 1, 0] + list(range(2, min(n, 4))) + [1])
