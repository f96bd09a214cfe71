"""BASELINE config 5 (Jacobi fp32, N = 2^30 cells, T = 4096) on ONE B200: the P = 1 point of
its scaling series — the persistent kernel over the whole domain (8 GiB of state + work)
(development aid):  python tools/time_j5.py"""
import sys

import torch

sys.path.insert(0, ".")
import paper_conf_ppopp_baskaranbkrrs08_b200 as sp  # noqa: E402
import sp_inputs  # noqa: E402


def main():
    n, T = 1 << 30, 4096
    tt = int(sys.argv[1]) if len(sys.argv) > 1 else 128
    a = torch.from_numpy(sp_inputs.jacobi_input(n, seed=2008)).cuda()
    w = torch.empty_like(a)
    flags = torch.empty(sp.jacobi1d_plan(n, T, tt, 0)["tiles"] + 1, dtype=torch.int32, device="cuda")
    sp.jacobi1d_timetiled_fused(a, 256, tt, 0, work=w, flags=flags)  # warm-up (4 passes)
    torch.cuda.synchronize()
    times = []
    for _ in range(2):
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        e0.record()
        sp.jacobi1d_timetiled_fused(a, T, tt, 0, work=w, flags=flags)
        e1.record()
        torch.cuda.synchronize()
        times.append(e0.elapsed_time(e1))
    t = min(times)
    ups = (n - 2) * T / (t * 1e-3)
    flops = 3 * ups
    print(f"J5 on 1 GPU: N=2^30 T={T} Tt={tt}: {t:.1f} ms (runs {', '.join(f'{x:.1f}' for x in times)})  "
          f"{ups / 1e12:.2f}e12 point-updates/s  {flops / 1e12:.1f} TFLOP/s fp32 "
          f"({flops / 37.22e12 * 100:.1f} % of 37.2)")


if __name__ == "__main__":
    main()
