"""Cluster-resident Jacobi latency by shape (development aid): J1 (N = 4,096, T = 64) per call
under CUDA-graph replay, and per-step time at T = 4,096 for a few N.  Shape via
$SP_JACOBI_RESIDENT (small / large; unset = library default)."""
import os
import sys

import numpy as np
import torch

sys.path.insert(0, ".")
import oracle  # noqa: E402
import paper_conf_ppopp_baskaranbkrrs08_b200 as sp  # noqa: E402
import sp_inputs  # noqa: E402


def graph_time(fn, reps=200):
    s = torch.cuda.Stream()
    with torch.cuda.stream(s):
        for _ in range(3):
            fn()
    torch.cuda.synchronize()
    g = torch.cuda.CUDAGraph()
    with torch.cuda.graph(g, stream=s):
        for _ in range(20):
            fn()
    g.replay()
    torch.cuda.synchronize()
    a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    a.record()
    for _ in range(reps // 20):
        g.replay()
    b.record()
    torch.cuda.synchronize()
    return a.elapsed_time(b) * 1e3 / reps


shape = os.environ.get("SP_JACOBI_RESIDENT", "default")
for n, T in [(4096, 64), (1700, 4096), (4096, 4096), (8064, 4096)]:
    a0 = sp_inputs.jacobi_input(n)
    x = torch.from_numpy(a0).cuda()
    y = torch.empty_like(x)
    try:
        sp.jacobi1d_resident(x, T, out=y)
    except Exception as ex:  # noqa: BLE001
        print(f"{shape} N={n} T={T}: {ex}")
        continue
    torch.cuda.synchronize()
    ok = np.array_equal(y.cpu().numpy(), oracle.jacobi1d(a0, T)) if T <= 64 else None
    us = graph_time(lambda: sp.jacobi1d_resident(x, T, out=y))
    print(f"{shape} N={n} T={T}: {us:.1f} us per call ({us * 1e3 / T:.0f} ns per step)  parity={ok}", flush=True)
