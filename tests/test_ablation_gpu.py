"""N1 ablation kernels (the paper's "GPU w/o scratchpad memory" versions)
compute the same results as the oracle, bit for bit."""
import numpy as np
import pytest
import torch

import oracle
import paper_conf_ppopp_baskaranbkrrs08_b200 as sp
import sp_inputs

pytestmark = pytest.mark.gpu


@pytest.mark.parametrize("n,steps", [(3, 5), (4096, 64), (10007, 33)])
def test_jacobi_untiled_equals_oracle(n, steps):
    a = sp_inputs.jacobi_input(n, seed=n)
    d = torch.from_numpy(a.copy()).cuda()
    sp.jacobi1d_untiled(d, steps)
    torch.cuda.synchronize()
    assert np.array_equal(d.cpu().numpy().view(np.uint32), oracle.jacobi1d(a, steps).view(np.uint32))


@pytest.mark.parametrize("W,H,R", [(64, 48, 5), (352, 288, 16), (130, 70, 32)])
def test_me_direct_equals_oracle(W, H, R):
    pitch = (W + 3) // 4 * 4
    fr = sp_inputs.me_sequence(2, W, H, R, seed=3, pitch=pitch)
    d = torch.from_numpy(fr).cuda()
    mv, sad, surf = sp.me_sad_search_direct(d[:-1], d[1:], W, H, R, with_surface=True)
    torch.cuda.synchronize()
    omv, osad, osurf = oracle.me_search(fr[0], fr[1], W, H, R, with_surface=True)
    assert np.array_equal(mv[0].cpu().numpy().reshape(-1, 2), omv)
    assert np.array_equal(sad[0].cpu().numpy().view(np.uint32).reshape(-1), osad)
    assert np.array_equal(surf[0].cpu().numpy().view(np.uint32).reshape(osurf.shape), osurf)
