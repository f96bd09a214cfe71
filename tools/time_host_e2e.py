"""sp_jacobi1d_host on J3 (2^26 cells, T = 1,024) at a few time tiles, both input routes
(development aid; skew via $SP_JACOBI_SKEW)."""
import os
import sys

import torch

sys.path.insert(0, ".")
import paper_conf_ppopp_baskaranbkrrs08_b200 as sp  # noqa: E402
import sp_inputs  # noqa: E402

n, T = 1 << 26, 1024
tts = [int(x) for x in sys.argv[1].split(",")] if len(sys.argv) > 1 else [128]
hh = torch.from_numpy(sp_inputs.jacobi_input(n)).pin_memory()
for tt in tts:
    for direct in (False, True):
        ctx = sp.Jacobi1DHost(n, T, tt, direct_input=direct)
        ctx.run(hh)
        torch.cuda.synchronize()
        ts = []
        for _ in range(4):
            a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            a.record()
            ctx.run(hh)
            b.record()
            torch.cuda.synchronize()
            ts.append(a.elapsed_time(b))
        print(f"skew={os.environ.get('SP_JACOBI_SKEW', 'default')} Tt={tt} "
              f"{'direct' if direct else 'copy-engine'}: {min(ts):.3f} ms", flush=True)
