import sys, torch
sys.path.insert(0, '.')
import paper_conf_ppopp_baskaranbkrrs08_b200 as sp, sp_inputs
n = 1 << 26
a = torch.from_numpy(sp_inputs.jacobi_input(n)).cuda()
w = torch.empty_like(a); fl = torch.empty(n, dtype=torch.int32, device='cuda')
if sys.argv[1] == 'fused':
    sp.jacobi1d_timetiled_fused(a, 128, 64, 0, work=w, flags=fl)
else:
    sp.jacobi1d_timetiled(a, 128, 64, 0, work=w)
torch.cuda.synchronize()
