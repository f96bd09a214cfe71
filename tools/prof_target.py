"""Minimal launch sequence of one kernel at the bench configuration, for ncu captures:
   python tools/prof_target.py jacobi [Tt] | jacobi_fused [Tt] | me | me16"""
import sys

import torch

sys.path.insert(0, ".")
import paper_conf_ppopp_baskaranbkrrs08_b200 as sp  # noqa: E402
import sp_inputs  # noqa: E402

what = sys.argv[1]
if what == "jacobi_fused":  # the bench's N = 1 launch: all T = 1024 steps in one persistent kernel
    tt = int(sys.argv[2]) if len(sys.argv) > 2 else 64
    n = 1 << 26
    a = torch.from_numpy(sp_inputs.jacobi_input(n)).cuda()
    w = torch.empty_like(a)
    for _ in range(2):
        sp.jacobi1d_timetiled_fused(a, 1024, tt, 0, work=w)
elif what == "jacobi":
    tt = int(sys.argv[2]) if len(sys.argv) > 2 else 64
    n = 1 << 26
    a = torch.from_numpy(sp_inputs.jacobi_input(n)).cuda()
    w = torch.empty_like(a)
    sp.jacobi1d_timetiled(a, 4 * tt, tt, 0, work=w)  # 4 launches
elif what == "me16":  # the R = 16 kernel at throughput: 256 CIF pairs (tools/time_me_r16.py)
    W, H, R = 352, 288, 16
    fr = torch.from_numpy(sp_inputs.me_sequence(257, W, H, R)).cuda()
    for _ in range(2):
        sp.me_search_sequence(fr, W, H, R)
else:
    W, H, R = 1920, 1080, 32
    fr = torch.from_numpy(sp_inputs.me_sequence(65, W, H, R)).cuda()  # the bench launch: 64 pairs
    for _ in range(2):
        sp.me_search_sequence(fr, W, H, R)
torch.cuda.synchronize()
print("done")
