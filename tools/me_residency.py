"""CTA residency of the persistent ME kernel: CTAs per SM and start / end spread (development
aid; python tools/build_exp.py res -DSP_ME_EXP=32, SP_LIB=tools/libsp_exp_res.so)."""
import collections
import ctypes
import sys

import numpy as np
import torch

sys.path.insert(0, ".")
import paper_conf_ppopp_baskaranbkrrs08_b200 as sp  # noqa: E402
import sp_inputs  # noqa: E402

W, H, R = 1920, 1080, 32
fr = torch.from_numpy(sp_inputs.me_sequence(65, W, H, R)).cuda()
buf = (ctypes.c_ulonglong * (4096 * 3))()
for rep in range(3):
    sp.me_search_sequence(fr, W, H, R)
    torch.cuda.synchronize()
assert sp.lib.sp_me_cta_read(buf) == 0
a = np.frombuffer(buf, dtype=np.uint64).reshape(4096, 3)[:592].astype(np.int64)
per_sm = collections.Counter(a[:, 0].tolist())
print("SMs used", len(per_sm), "CTAs per SM histogram", collections.Counter(per_sm.values()))
t0 = a[:, 1].min()
st, en = (a[:, 1] - t0) / 1e3, (a[:, 2] - t0) / 1e3
print(f"start us: min {st.min():.1f} max {st.max():.1f} p50 {np.median(st):.1f}; end us: min {en.min():.1f} "
      f"p50 {np.median(en):.1f} max {en.max():.1f}")
print("latest starters:", sorted(zip(st.tolist(), a[:, 0].tolist()))[-8:])
