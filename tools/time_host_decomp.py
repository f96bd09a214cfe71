"""Where the end-to-end Jacobi host path's time goes (development aid): J3 (2^26 cells, T =
1,024, Tt = 128) through sp_jacobi1d_timetiled_stream with each end in device or pinned host
memory (wavefront skew 512), the host call itself, and plain copy-engine transfers."""
import sys

import torch

sys.path.insert(0, ".")
import paper_conf_ppopp_baskaranbkrrs08_b200 as sp  # noqa: E402
import sp_inputs  # noqa: E402

n, T, Tt = 1 << 26, 1024, 128
skews = [int(x) for x in sys.argv[1].split(",")] if len(sys.argv) > 1 else [512]
a0 = torch.from_numpy(sp_inputs.jacobi_input(n))
hin = a0.clone().pin_memory()
hout = torch.empty(n, dtype=torch.float32).pin_memory()
din = a0.cuda()
dout = torch.empty(n, dtype=torch.float32, device="cuda")
b0 = torch.empty_like(din)
b1 = torch.empty_like(din)
fl = torch.empty(sp.jacobi1d_plan(n, T, Tt, 0)["tiles"] + 1, dtype=torch.int32, device="cuda")


def ev(fn, reps=4):
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
    return min(ts)


for D in skews:
    for name, i, o in [("dev->dev", din, dout), ("host->dev", hin, dout), ("dev->host", din, hout),
                       ("host->host", hin, hout)]:
        t = ev(lambda: sp.jacobi1d_timetiled_stream(i, o, T, Tt, 0, skew=D, buf0=b0, buf1=b1, flags=fl))
        print(f"stream {name:10s} D={D}: {t:.3f} ms", flush=True)
hh = a0.clone().pin_memory()
for direct in (False, True):
    ctx = sp.Jacobi1DHost(n, T, Tt, direct_input=direct)
    print(f"sp_jacobi1d_host ({'direct PCIe move-in' if direct else 'copy-engine input'}): "
          f"{ev(lambda: ctx.run(hh)):.3f} ms", flush=True)
s2 = torch.cuda.Stream()
print(f"H2D copy 256 MiB: {ev(lambda: din.copy_(hin, non_blocking=True)):.3f} ms", flush=True)
print(f"D2H copy 256 MiB: {ev(lambda: hout.copy_(dout, non_blocking=True)):.3f} ms", flush=True)


def both():
    ev0 = torch.cuda.Event()
    ev0.record()
    s2.wait_event(ev0)
    din.copy_(hin, non_blocking=True)
    with torch.cuda.stream(s2):
        hout.copy_(dout, non_blocking=True)
    torch.cuda.current_stream().wait_stream(s2)


print(f"H2D + D2H concurrent: {ev(both):.3f} ms", flush=True)
