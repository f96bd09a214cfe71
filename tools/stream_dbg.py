"""Wait / stall counters of the persistent Jacobi under pass-major vs wavefront order
(needs the SP_JAC_DEBUG build: python tools/build_exp.py dbg -DSP_JAC_DEBUG, SP_LIB=...)."""
import ctypes
import sys

import torch

sys.path.insert(0, ".")
import paper_conf_ppopp_baskaranbkrrs08_b200 as sp  # noqa: E402
import sp_inputs  # noqa: E402

n, T, tt = 1 << 26, 1024, 64
a0 = torch.from_numpy(sp_inputs.jacobi_input(n)).cuda()
a = torch.empty_like(a0)
w = torch.empty_like(a0)
fl = torch.empty(n // 64, dtype=torch.int32, device="cuda")
buf = (ctypes.c_ulonglong * 16)()
sp.lib.sp_jac_dbg_read.argtypes = [ctypes.c_void_p]
for skew in [int(x) for x in (sys.argv[1] if len(sys.argv) > 1 else "0,512,2048").split(",")]:
    for rep in range(2):
        sp.lib.sp_jac_dbg_read(buf)
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        e0.record()
        sp.jacobi1d_timetiled_stream(a0, a, T, tt, 0, skew, buf0=a, buf1=w, flags=fl)
        e1.record()
        torch.cuda.synchronize()
    sp.lib.sp_jac_dbg_read(buf)
    t0, t1 = max(1, buf[8]), max(1, buf[9])
    print(f"skew {skew}: {e0.elapsed_time(e1):.3f} ms; tiles p0/p>0 {buf[8]} {buf[9]}; "
          f"prefetch cyc/tile {buf[4] // t0} {buf[5] // t1}; steps cyc/tile {buf[6] // t0} {buf[7] // t1}; "
          f"pending waits {buf[0]} avg {buf[1] / max(1, buf[0]):.0f} cyc; "
          f"mbar wait cyc/tile p0 {buf[3] // t0} p>0 {buf[2] // t1}", flush=True)
