"""The latency-bound BASELINE configs 1 and 2 on one B200 (development aid):
J1 = Jacobi N = 4096, T = 64, Tt = 16 through the persistent pass kernel and the
cluster-resident kernel; M2 = one CIF pair, +-16 (full surface off / on)."""
import os
import sys

import numpy as np
import torch

sys.path.insert(0, ".")
import paper_conf_ppopp_baskaranbkrrs08_b200 as sp  # noqa: E402
import sp_inputs  # noqa: E402


def ev_time(fn, reps=20, warm=5):
    for _ in range(warm):
        fn()
    torch.cuda.synchronize()
    ts = []
    for _ in range(reps):
        a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        a.record()
        fn()
        b.record()
        torch.cuda.synchronize()
        ts.append(a.elapsed_time(b) * 1e3)
    return min(ts), float(np.median(ts))


def main():
    a0 = torch.from_numpy(sp_inputs.jacobi_input(4096, seed=2008)).cuda()
    a, w = a0.clone(), torch.empty_like(a0)
    fl = torch.empty(64, dtype=torch.int32, device="cuda")
    def persistent():  # (the fused call's default route below Tt = 32 is per-pass launches)
        os.environ["SP_JACOBI_FUSED_PERSISTENT"] = "1"
        sp.jacobi1d_timetiled_fused(a, 64, 16, 512, work=w, flags=fl)
        del os.environ["SP_JACOBI_FUSED_PERSISTENT"]

    for name, fn in [("J1 persistent pass kernel (Tt 16, S 512)", persistent),
                     ("J1 per-pass launches (Tt 16, S 512)", lambda: sp.jacobi1d_timetiled(a, 64, 16, 512, work=w)),
                     ("J1 cluster-resident", lambda: sp.jacobi1d_resident(a0, 64, out=a))]:
        b, m = ev_time(fn)
        print(f"{name}: best {b:.1f} us, median {m:.1f} us  ({4094 * 64 / (b * 1e-6) / 1e9:.1f} GUpd/s)")
    res = sp.jacobi1d_resident_prepared(a0, 64, out=a)
    b, m = ev_time(res)
    print(f"J1 cluster-resident, prepared call: best {b:.1f} us, median {m:.1f} us")
    fr = torch.from_numpy(sp_inputs.me_sequence(2, 352, 288, 16)).cuda()
    pm = sp.me_search_prepared(fr, 352, 288, 16)
    b, m = ev_time(pm)
    print(f"M2 CIF +-16, 1 pair, prepared call: best {b:.1f} us, median {m:.1f} us ({390028 / (b * 1e-6) / 1e9:.1f} GSAD/s)")
    for surf in (False, True):
        b, m = ev_time(lambda: sp.me_search_sequence(fr, 352, 288, 16, with_surface=surf))
        print(f"M2 CIF +-16, 1 pair{' + full surface' if surf else ''}: best {b:.1f} us, median {m:.1f} us "
              f"({390028 / (b * 1e-6) / 1e9:.1f} GSAD/s)")


def graph_time(fn, reps=50):
    """device time per call: the call captured once in a CUDA graph, replayed back to back"""
    s = torch.cuda.Stream()
    s.wait_stream(torch.cuda.current_stream())
    with torch.cuda.stream(s):
        fn()
    torch.cuda.current_stream().wait_stream(s)
    torch.cuda.synchronize()
    g = torch.cuda.CUDAGraph()
    with torch.cuda.graph(g):
        fn()
    g.replay()
    torch.cuda.synchronize()
    a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    a.record()
    for _ in range(reps):
        g.replay()
    b.record()
    torch.cuda.synchronize()
    return a.elapsed_time(b) * 1e3 / reps


def graphs():
    a0 = torch.from_numpy(sp_inputs.jacobi_input(4096, seed=2008)).cuda()
    a = torch.empty_like(a0)
    print(f"[graph] J1 cluster-resident: {graph_time(lambda: sp.jacobi1d_resident(a0, 64, out=a)):.1f} us per call")
    fr = torch.from_numpy(sp_inputs.me_sequence(2, 352, 288, 16)).cuda()
    out = (torch.empty((1, 18, 22, 2), dtype=torch.int16, device="cuda"),
           torch.empty((1, 18, 22), dtype=torch.int32, device="cuda"), None)
    print(f"[graph] M2 CIF +-16, 1 pair: {graph_time(lambda: sp.me_search_sequence(fr, 352, 288, 16, out=out)):.1f} us per call")


if __name__ == "__main__":
    graphs()
    main()
