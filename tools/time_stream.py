"""Device timing of the persistent Jacobi at J3 under different unit orders (skew) and of the
end-to-end host-buffer path (development aid):
   python tools/time_stream.py [Tt,...] [--skews 0,256,...] [--host]"""
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


def arg(name, default):
    for x in sys.argv[1:]:
        if x.startswith(name + "="):
            return x.split("=", 1)[1]
    return default


def main():
    n, T = 1 << 26, 1024
    a0 = torch.from_numpy(sp_inputs.jacobi_input(n)).cuda()
    a = a0.clone()
    w = torch.empty_like(a)
    flags = torch.empty(n // 64, dtype=torch.int32, device="cuda")
    tts = [int(x) for x in arg("--tt", "64").split(",")]
    skews = [int(x) for x in arg("--skews", "0,256").split(",")]
    for tt in tts:
        for skew in skews:
            def run():
                sp.jacobi1d_timetiled_stream(a0, a, T, tt, 0, skew, buf0=a, buf1=w, flags=flags)
            best, med = ev_time(run)
            ups = (n - 2) * T / (best * 1e-3)
            print(f"jacobi J3 Tt={tt} skew={skew}: best {best:.3f} ms  med {med:.3f}  {ups/1e9:.1f} GUpd/s", flush=True)
        if "--host" in sys.argv:
            h = torch.from_numpy(sp_inputs.jacobi_input(n)).pin_memory()
            ctx = sp.Jacobi1DHost(n, T, tt)
            best, med = ev_time(lambda: ctx.run(h))
            t0 = time.perf_counter()
            for _ in range(3):
                ctx.run(h)
            torch.cuda.synchronize()
            wall = (time.perf_counter() - t0) / 3 * 1e3
            print(f"jacobi host e2e Tt={tt}: events best {best:.3f} ms med {med:.3f}; wall {wall:.3f} ms "
                  f"-> {(n - 2) * T / (wall * 1e-3) / 1e9:.1f} GUpd/s", flush=True)
            # the old e2e recipe for reference: pinned H2D, device run, D2H
            d = torch.empty(n, dtype=torch.float32, device="cuda")
            o = torch.empty(n, dtype=torch.float32).pin_memory()

            def old():
                d.copy_(h, non_blocking=True)
                sp.jacobi1d_timetiled_fused(d, T, tt, 0, work=w, flags=flags)
                o.copy_(d, non_blocking=True)
            best, med = ev_time(old)
            print(f"jacobi copy+run+copy Tt={tt}: best {best:.3f} ms", flush=True)


if __name__ == "__main__" and "--me" not in sys.argv:
    main()


def me_main():
    W, H, R, F = 1920, 1080, 32, 65
    fr = sp_inputs.me_sequence(F, W, H, R)
    h = torch.from_numpy(fr).pin_memory()
    d = h.cuda()
    ctx = sp.MESearchHost(F, W, H, fr.shape[2], R)
    best, med = ev_time(lambda: sp.me_search_sequence(d, W, H, R), reps=3)
    print(f"ME device-resident: best {best:.3f} ms", flush=True)
    best, med = ev_time(lambda: ctx.run(h), reps=3)
    t0 = time.perf_counter()
    for _ in range(3):
        ctx.run(h)
    torch.cuda.synchronize()
    wall = (time.perf_counter() - t0) / 3 * 1e3
    print(f"ME host e2e: events best {best:.3f} ms; wall {wall:.3f} ms -> {32934600 * 64 / (wall * 1e-3) / 1e9:.1f} GSAD/s",
          flush=True)
    t0 = time.perf_counter()
    for _ in range(3):
        dd = h.to("cuda", non_blocking=True)
        mv, sad, _ = sp.me_search_sequence(dd, W, H, R)
        mv.cpu(), sad.cpu()
    torch.cuda.synchronize()
    print(f"ME copy+run+copy wall {(time.perf_counter() - t0) / 3 * 1e3:.3f} ms", flush=True)


if __name__ == "__main__" and "--me" in sys.argv:
    me_main()
