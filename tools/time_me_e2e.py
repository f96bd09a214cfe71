"""M4 (64 pairs of 1080p, +-32) through sp_me_search_host from pinned host frames vs the
device-resident search (development aid)."""
import sys

import torch

sys.path.insert(0, ".")
import paper_conf_ppopp_baskaranbkrrs08_b200 as sp  # noqa: E402
import sp_inputs  # noqa: E402

W, H, R, F = 1920, 1080, 32, 65
fr = sp_inputs.me_sequence(F, W, H, R)
h = torch.from_numpy(fr).pin_memory()
d = h.cuda()
ctx = sp.MESearchHost(F, W, H, fr.shape[2], R)


def ev(fn, reps=5):
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


print(f"M4 device-resident: {ev(lambda: sp.me_search_sequence(d, W, H, R)):.3f} ms", flush=True)
print(f"M4 sp_me_search_host: {ev(lambda: ctx.run(h)):.3f} ms", flush=True)
