import sys, torch, ctypes
sys.path.insert(0, '.')
import paper_conf_ppopp_baskaranbkrrs08_b200 as sp, sp_inputs
n = 1 << 26
a = torch.from_numpy(sp_inputs.jacobi_input(n)).cuda()
w = torch.empty_like(a); fl = torch.empty(n, dtype=torch.int32, device='cuda')
buf = (ctypes.c_ulonglong * 16)()
for steps in (64, 128, 256, 1024):
    sp.jacobi1d_timetiled_fused(a, steps, 64, 0, work=w, flags=fl); torch.cuda.synchronize()
    sp.lib.sp_jac_dbg_read(buf)
    t0, t1 = max(1, buf[8]), max(1, buf[9])
    print(steps, 'tiles p0/p>0', buf[8], buf[9], 'prefetch cyc/tile', buf[4] // t0, buf[5] // t1, 'steps cyc/tile', buf[6] // t0, buf[7] // t1, flush=True)
    print('   boundary p0/p>0', buf[10], buf[11], 'sum h', buf[12], buf[13])
    print('   pending waits', buf[0], 'avg cycles', buf[1] / max(1, buf[0]), 'mbar wait/warp p0', buf[3] / 2368, 'p>0', buf[2] / 2368)
