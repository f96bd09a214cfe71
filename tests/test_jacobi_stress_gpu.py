"""Schedule stress of the persistent Jacobi: a build with SP_JAC_STRESS makes
one tile in eight (a hash of tile and pass) finish 20 us late, so tiles of the next pass
really wait on their dependence flags, warps publish before waiting, and the wavefront and
host-memory orders run with stragglers.  Results must stay bit-identical to the oracle."""
import os
import subprocess
import sys

import numpy as np
import pytest

import oracle
import sp_inputs

pytestmark = pytest.mark.gpu

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
CASES = [(40011, 150, 16, 8), (100003, 97, 64, 0), (30000, 64, 32, 100), (7777, 200, 3, 4)]

CHILD = r"""
import sys
import numpy as np
import torch
sys.path.insert(0, sys.argv[1])
import paper_conf_ppopp_baskaranbkrrs08_b200 as sp
import sp_inputs
out = {}
for k, (n, steps, tt, S) in enumerate(eval(sys.argv[3])):
    a0 = sp_inputs.jacobi_input(n, seed=77 + k)
    d = torch.from_numpy(a0.copy()).cuda()
    sp.jacobi1d_timetiled_fused(d, steps, tt, S)
    o = torch.empty_like(d)
    sp.jacobi1d_timetiled_stream(torch.from_numpy(a0.copy()).cuda(), o, steps, tt, S, 64)
    h = torch.from_numpy(a0.copy()).pin_memory()
    sp.Jacobi1DHost(n, steps, tt, S).run(h)
    torch.cuda.synchronize()
    out[f"f{k}"], out[f"w{k}"], out[f"h{k}"] = d.cpu().numpy(), o.cpu().numpy(), h.numpy().copy()
np.savez(sys.argv[2], **out)
"""


def _stress_lib():
    lib = os.path.join(ROOT, "tools", "libsp_exp_jstress.so")
    src = os.path.join(ROOT, "paper_conf_ppopp_baskaranbkrrs08_b200", "csrc", "jacobi.cu")
    if not os.path.exists(lib) or os.path.getmtime(lib) < os.path.getmtime(src):
        subprocess.check_call([sys.executable, os.path.join(ROOT, "tools", "build_exp.py"), "jstress",
                               "-DSP_JAC_STRESS"], cwd=ROOT, stdout=subprocess.DEVNULL)
    return lib


def test_stragglers_keep_the_persistent_orders_exact(tmp_path):
    out = str(tmp_path / "jstress.npz")
    env = dict(os.environ, SP_LIB=_stress_lib(), SP_JACOBI_FUSED_PERSISTENT="1")  # (persistent at every Tt)
    subprocess.check_call([sys.executable, "-c", CHILD, ROOT, out, repr(CASES)], env=env, cwd=ROOT, timeout=600)
    got = np.load(out)
    for k, (n, steps, tt, S) in enumerate(CASES):
        want = oracle.jacobi1d(sp_inputs.jacobi_input(n, seed=77 + k), steps).view(np.uint32)
        for tag, name in (("f", "persistent pass-major"), ("w", "wavefront"), ("h", "host memory")):
            assert np.array_equal(got[f"{tag}{k}"].view(np.uint32), want), (name, n, steps, tt, S)
