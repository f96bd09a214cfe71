import sys, torch, time
sys.path.insert(0, '.')
import paper_conf_ppopp_baskaranbkrrs08_b200 as sp, sp_inputs, oracle, numpy as np
n = 1 << 26
a0 = torch.from_numpy(sp_inputs.jacobi_input(n)).cuda()
w = torch.empty_like(a0); fl = torch.empty(n, dtype=torch.int32, device='cuda')
for steps in (64, 128, 256, 1024):
    for fused in (False, True):
        a = a0.clone()
        f = (lambda: sp.jacobi1d_timetiled_fused(a, steps, 64, 0, work=w, flags=fl)) if fused else (lambda: sp.jacobi1d_timetiled(a, steps, 64, 0, work=w))
        f(); torch.cuda.synchronize()
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        e0.record(); f(); e1.record(); torch.cuda.synchronize()
        print(steps, 'fused' if fused else 'pass ', round(e0.elapsed_time(e1), 3), 'ms', flush=True)
a = sp_inputs.jacobi_input(4096, seed=2008)
want = oracle.jacobi1d(a, 64)
for S in (0, 256, 16):
    d = torch.from_numpy(a.copy()).cuda(); sp.jacobi1d_timetiled_fused(d, 64, 16, S); torch.cuda.synchronize()
    g = d.cpu().numpy(); bad = np.nonzero(g.view(np.uint32) != want.view(np.uint32))[0]
    print('J1 S', S, 'mismatches', bad.size, bad[:10])
