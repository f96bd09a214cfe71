import sys, torch
sys.path.insert(0, ".")
import paper_conf_ppopp_baskaranbkrrs08_b200 as sp, sp_inputs
def ev(fn, reps=5):
    fn(); torch.cuda.synchronize()
    best = 1e9
    for _ in range(reps):
        a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        a.record(); fn(); b.record(); torch.cuda.synchronize(); best = min(best, a.elapsed_time(b))
    return best
for n in [3, 1700, 8192, 32768, 200000]:
    a = torch.from_numpy(sp_inputs.jacobi_input(n, seed=1)).cuda()
    row = []
    for steps in [1, 14, 15, 28, 140, 1400, 4096]:
        row.append(f"{steps}:{ev(lambda: sp.jacobi1d_resident(a, steps))*1e3:.0f}us")
    print(n, " ".join(row), flush=True)
