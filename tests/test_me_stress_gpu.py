"""Race stress of the ME kernel's shared-memory pipeline: a build with
SP_ME_EXP=64 delays the upper half of each CTA's warps by 20 us per macroblock, so the lower
warps build the NEXT macroblock's byte-phase copies (the other stage) while the upper ones
still read this one's.  Any overlap between the two stages' shared-memory regions then
corrupts SADs deterministically instead of rarely.  (It caught one: stage 0's phase-3 copy
and stage 1's phase-1 copy shared 64 bytes, see MeGeom::kSlot.)  Full SAD surfaces of the
device path and MV / SAD of the host-buffer path are compared with the oracle."""
import os
import subprocess
import sys

import numpy as np
import pytest

import oracle
import sp_inputs

pytestmark = pytest.mark.gpu

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
W, H, R, F = 352, 288, 32, 4

CHILD = r"""
import sys
import numpy as np
import torch
sys.path.insert(0, sys.argv[1])
import paper_conf_ppopp_baskaranbkrrs08_b200 as sp
import sp_inputs
W, H, R, F = (int(x) for x in sys.argv[3:7])
fr = sp_inputs.me_sequence(F, W, H, R)
mv, sad, surf = sp.me_search_sequence(torch.from_numpy(fr).cuda(), W, H, R, with_surface=True)
ctx = sp.MESearchHost(F, W, H, fr.shape[2], R)
hmv, hsad = ctx.run(torch.from_numpy(fr).pin_memory())
torch.cuda.synchronize()
np.savez(sys.argv[2], mv=mv.cpu().numpy(), sad=sad.cpu().numpy(), surf=surf.cpu().numpy(),
         hmv=hmv.numpy(), hsad=hsad.numpy())
"""


def _stress_lib():
    if os.environ.get("SP_ME_STRESS_LIB"):  # a prebuilt variant (e.g. to show the test fails on a bad layout)
        return os.environ["SP_ME_STRESS_LIB"]
    lib = os.path.join(ROOT, "tools", "libsp_exp_stress.so")
    src = os.path.join(ROOT, "paper_conf_ppopp_baskaranbkrrs08_b200", "csrc", "me.cu")
    if not os.path.exists(lib) or os.path.getmtime(lib) < os.path.getmtime(src):
        subprocess.check_call([sys.executable, os.path.join(ROOT, "tools", "build_exp.py"), "stress", "-DSP_ME_EXP=64"],
                              cwd=ROOT, stdout=subprocess.DEVNULL)
    return lib


def test_delayed_warps_do_not_corrupt_the_other_stage(tmp_path):
    out = str(tmp_path / "stress.npz")
    env = dict(os.environ, SP_LIB=_stress_lib())
    subprocess.check_call([sys.executable, "-c", CHILD, ROOT, out, str(W), str(H), str(R), str(F)], env=env,
                          cwd=ROOT, timeout=600)
    got = np.load(out)
    fr = sp_inputs.me_sequence(F, W, H, R)
    side = 2 * R + 1
    for p in range(F - 1):
        omv, osad, osurf = oracle.me_search(fr[p], fr[p + 1], W, H, R, with_surface=True)
        surf = got["surf"][p].reshape(-1, side * side).view(np.uint32)
        assert np.array_equal(surf, osurf), f"pair {p}: SAD surface differs at {np.argwhere(surf != osurf)[:5]}"
        assert np.array_equal(got["mv"][p].reshape(-1, 2), omv)
        assert np.array_equal(got["sad"][p].reshape(-1).view(np.uint32), osad)
        assert np.array_equal(got["hmv"][p].reshape(-1, 2), omv)
        assert np.array_equal(got["hsad"][p].reshape(-1).view(np.uint32), osad)
