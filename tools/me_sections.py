"""Per-section cycle split of the ME kernel (development aid; needs a library built with
    python tools/build_exp.py prof -DSP_ME_EXP=16   and   SP_LIB=tools/libsp_exp_prof.so)."""
import ctypes
import sys

import torch

sys.path.insert(0, ".")
import paper_conf_ppopp_baskaranbkrrs08_b200 as sp  # noqa: E402
import sp_inputs  # noqa: E402

NAMES = ["tma wait", "phase build", "B1+finalize", "main loop", "corner", "-", "-", "epilogue"]
W, H, R = 1920, 1080, 32
fr = torch.from_numpy(sp_inputs.me_sequence(65, W, H, R)).cuda()
buf = (ctypes.c_ulonglong * 8)()
for rep in range(3):
    sp.me_search_sequence(fr, W, H, R)
    torch.cuda.synchronize()
    assert sp.lib.sp_me_prof_read(buf) == 0
mbs = 64 * (W // 16) * (H // 16)
warps = 4
tot = sum(buf)
for k, n in enumerate(NAMES):
    print(f"{n:14s} {buf[k] / (mbs * warps):9.0f} cycles/MB/warp  {100 * buf[k] / tot:5.1f} %")
print(f"{'total':14s} {tot / (mbs * warps):9.0f}")
