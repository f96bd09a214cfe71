"""Quick device timing of the two kernels at the bench configurations (development aid)."""
import sys
import time

import numpy as np
import torch

sys.path.insert(0, ".")
import paper_conf_ppopp_baskaranbkrrs08_b200 as sp  # noqa: E402
import sp_inputs  # noqa: E402


def ev_time(fn, reps=5, warm=2):
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
        ts.append(a.elapsed_time(b))
    return min(ts), float(np.median(ts))


def main():
    n, T = 1 << 26, 1024
    a0 = torch.from_numpy(sp_inputs.jacobi_input(n)).cuda()
    a = a0.clone()
    w = torch.empty_like(a)
    flags = torch.empty(n, dtype=torch.int32, device="cuda")
    pos = [x for x in sys.argv[1:] if not x.startswith("--")]
    for tt in ([] if "--me-only" in sys.argv else [int(x) for x in (pos[0].split(",") if pos else ["16", "32"])]):
        def run():
            a.copy_(a0)
            if "--fused" in sys.argv:
                sp.jacobi1d_timetiled_fused(a, T, tt, 0, work=w, flags=flags)
            else:
                sp.jacobi1d_timetiled(a, T, tt, 0, work=w)
        copy_ms, _ = ev_time(lambda: a.copy_(a0))
        best, med = ev_time(run)
        t = best - copy_ms
        ups = (n - 2) * T / (t * 1e-3)
        print(f"jacobi N=2^26 T={T} Tt={tt}: {t:.3f} ms  {ups/1e9:.1f} GUpd/s  "
              f"HBM-alg {8.0*(n)*(T/tt)/(t*1e-3)/1e9:.0f} GB/s  plan={sp.jacobi1d_plan(n, T, tt, 0)}", flush=True)
    if '--no-me' in sys.argv:
        return
    W, H, R, F = 1920, 1080, 32, 65
    t0 = time.time()
    fr = torch.from_numpy(sp_inputs.me_sequence(F, W, H, R)).cuda()
    print(f"gen {time.time()-t0:.1f}s", flush=True)
    out = None

    def me():
        nonlocal out
        out = sp.me_search_sequence(fr, W, H, R)
    best, med = ev_time(me, reps=5)
    sads = 32934600 * 64
    print(f"ME 1080p R=32 64 pairs: {best:.3f} ms (med {med:.3f})  {sads/(best*1e-3)/1e9:.1f} GSAD/s  "
          f"{sads*256/(best*1e-3)/1e12:.1f} Tabsdiff/s", flush=True)


if __name__ == "__main__":
    main()
