"""Debug aid: R = 16 many-pair parity, listing the macroblocks that differ from the oracle."""
import sys
import numpy as np
import torch
sys.path.insert(0, ".")
import oracle  # noqa: E402
import paper_conf_ppopp_baskaranbkrrs08_b200 as sp  # noqa: E402
import sp_inputs  # noqa: E402

W, H, R, P = 352, 288, 16, int(sys.argv[1]) if len(sys.argv) > 1 else 24
fr = sp_inputs.me_sequence(P + 1, W, H, R, seed=77)
mv, sad, _ = sp.me_search_sequence(torch.from_numpy(fr).cuda(), W, H, R)
torch.cuda.synchronize()
mv, sad = mv.cpu().numpy(), sad.cpu().numpy().view(np.uint32)
bad = 0
for p in range(P):
    omv, osad, _ = oracle.me_search(fr[p], fr[p + 1], W, H, R, with_surface=False)
    g = mv[p].reshape(-1, 2)
    s = sad[p].reshape(-1)
    for k in np.nonzero((g != omv).any(1) | (s != osad))[0]:
        if bad < 20:
            print(f"pair {p} mb {k} (row {k // 22}, col {k % 22}): gpu mv {g[k]} sad {s[k]}  oracle mv {omv[k]} sad {osad[k]}")
        bad += 1
print("bad", bad, "of", P * 396)
