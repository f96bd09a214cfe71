import sys, numpy as np, torch
sys.path.insert(0, ".")
import paper_conf_ppopp_baskaranbkrrs08_b200 as sp, sp_inputs, oracle
cfg = [(64, 48, 5), (64, 48, 16), (352, 288, 16), (128, 96, 32)]
for W, H, R in cfg[int(sys.argv[1]) if len(sys.argv) > 1 else 0:]:
    fr = sp_inputs.me_sequence(2, W, H, R)
    d = torch.from_numpy(fr).cuda()
    try:
        mv, sad, surf = sp.me_search_sequence(d, W, H, R, with_surface=True)
        torch.cuda.synchronize()
        omv, osad, osurf = oracle.me_search(fr[0], fr[1], W, H, R, with_surface=True)
        print(W, H, R, "mv ok", np.array_equal(mv[0].cpu().numpy().reshape(-1, 2), omv),
              "sad ok", np.array_equal(sad[0].cpu().numpy().view(np.uint32).reshape(-1), osad), flush=True)
    except Exception as e:
        print(W, H, R, "ERR", e, flush=True)
        break
