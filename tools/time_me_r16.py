"""Throughput of the R = 16 ME kernel (BASELINE config 2's CIF +-16, batched so the GPU is
full): 256 CIF pairs, against the VABSDIFF4 roof (development aid)."""
import sys

import torch

sys.path.insert(0, ".")
import paper_conf_ppopp_baskaranbkrrs08_b200 as sp  # noqa: E402
import sp_inputs  # noqa: E402


def main():
    W, H, R, P = 352, 288, 16, 256
    fr = torch.from_numpy(sp_inputs.me_sequence(P + 1, W, H, R)).cuda()
    for _ in range(3):
        sp.me_search_sequence(fr, W, H, R)
    torch.cuda.synchronize()
    ts = []
    for _ in range(5):
        a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        a.record()
        sp.me_search_sequence(fr, W, H, R)
        b.record()
        torch.cuda.synchronize()
        ts.append(a.elapsed_time(b))
    t = min(ts)
    sads = 390028 * P
    roof = 148 * 64 * 4 * 1.965e9
    print(f"ME CIF +-16 x {P} pairs: {t:.3f} ms  {sads / t / 1e6:.1f} GSAD/s  "
          f"{sads * 256 / (t * 1e-3) / 1e12:.1f} Tabsdiff/s = {sads * 256 / (t * 1e-3) / roof * 100:.1f} % of the VABSDIFF4 roof")


if __name__ == "__main__":
    main()
