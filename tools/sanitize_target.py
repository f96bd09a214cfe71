"""Small invocations of every device entry point, for compute-sanitizer runs (T6)."""
import os
import sys

import torch

# a few ME CTAs walking many macroblocks each: racecheck then sees both pipeline stages of a CTA
os.environ.setdefault("SP_ME_GRID_CAP", "4")
os.environ.setdefault("SP_JACOBI_GRID_CAP", "2")  # likewise: many tiles per Jacobi warp
sys.path.insert(0, ".")
import paper_conf_ppopp_baskaranbkrrs08_b200 as sp  # noqa: E402
import sp_inputs  # noqa: E402


def mark(what):
    torch.cuda.synchronize()
    print(f"[sanitize] {what}", file=sys.stderr, flush=True)


a = torch.from_numpy(sp_inputs.jacobi_input(4099, seed=1)).cuda()
mark("sp.jacobi1d_timetiled")
sp.jacobi1d_timetiled(a, 37, 16, 256)
mark("sp.jacobi1d_timetiled")
sp.jacobi1d_timetiled(a, 20, 5, 0)
mark("sp.jacobi1d_timetiled_fused (persistent launch at every time tile)")
os.environ["SP_JACOBI_FUSED_PERSISTENT"] = "1"
sp.jacobi1d_timetiled_fused(a, 37, 16, 256)
sp.jacobi1d_timetiled_fused(a, 20, 5, 8)
mark("sp.jacobi1d_timetiled_fused (in-place geometry: Tt >= 48)")
sp.jacobi1d_timetiled_fused(a, 150, 64, 0)
sp.jacobi1d_timetiled_fused(a, 130, 48, 8)
del os.environ["SP_JACOBI_FUSED_PERSISTENT"]
mark("sp.jacobi1d_timetiled_fused (default route below Tt = 32: one launch per pass)")
sp.jacobi1d_timetiled_fused(a, 37, 16, 256)
mark("sp.jacobi1d_timetiled_stream (wavefront, device)")
o = torch.empty_like(a)
sp.jacobi1d_timetiled_stream(a, o, 37, 16, 256, 4)
sp.jacobi1d_timetiled_stream(a, o, 150, 64, 8, 64)
mark("sp.jacobi1d_host (pinned in/out, 3 passes)")
h = a.cpu().pin_memory()
sp.Jacobi1DHost(4099, 37, 16, 256).run(h)
mark("sp.jacobi1d_host (in place geometry, host-output instantiation)")
sp.Jacobi1DHost(4099, 150, 64, 8).run(h)
sp.Jacobi1DHost(4099, 150, 64, 0).run(h)
mark("sp.jacobi1d_host (1 pass: redirect + copy)")
sp.Jacobi1DHost(4099, 9, 16, 0).run(h)
mark("sp.jacobi1d_resident (one cluster, small and large shapes)")
sp.jacobi1d_resident(a, 45)
big = torch.from_numpy(sp_inputs.jacobi_input(150000, seed=2)).cuda()
sp.jacobi1d_resident(big, 33)
mark("sp.exec_block (Figure 1 program, tiled mat-vec with hoisting)")
from tests import exec_programs as X  # noqa: E402
blk, bodies, boxes, printed = X.figure1()
g = torch.Generator().manual_seed(0)
sp.exec_block(blk, bodies, [torch.randn(200, 200, generator=g).cuda(), torch.randn(200, 200, generator=g).cuda()])
blk, bodies, boxes, tiles = X.matvec(70, 100, 16)
sp.exec_block(blk, bodies, [torch.randn(70, generator=g).cuda(), torch.randn(70, 100, generator=g).cuda(),
                            torch.randn(100, generator=g).cuda()], tile_params=tiles, tiles_per_cta=7, hoist=True)
mark("sp.jacobi1d_untiled")
sp.jacobi1d_untiled(a, 3)
fr = torch.from_numpy(sp_inputs.me_sequence(3, 352, 288, 16)).cuda()
mark("sp.me_search_sequence")
sp.me_search_sequence(fr, 352, 288, 16, with_surface=True)
fr2 = torch.from_numpy(sp_inputs.me_sequence(2, 130, 70, 32, pitch=144)).cuda()
mark("sp.me_search_sequence")
sp.me_search_sequence(fr2, 130, 70, 32)
mark("sp.me_search_sequence")
sp.me_search_sequence(fr2, 130, 70, 5)
mark("sp.me_search_sequence_unrestricted")
sp.me_search_sequence_unrestricted(fr2, 130, 70, 32)
mark("sp.me_search_host (streamed frames, pinned outputs)")
sp.MESearchHost(3, 352, 288, fr.shape[2], 16).run(fr.cpu().pin_memory())
fr3 = torch.from_numpy(sp_inputs.me_sequence(2, 352, 288, 32)).cuda()
mark("sp.me_search_sequence (CIF +-32: 4-warp CTAs, two stages per CTA)")
sp.me_search_sequence(fr3, 352, 288, 32)
mark("sp.me_search_host (CIF +-32, streamed)")
sp.MESearchHost(2, 352, 288, fr3.shape[2], 32).run(fr3.cpu().pin_memory())
mark("sp.me_search_sequence (R = 16 class order with half-frame border searches, 4 CTAs)")
os.environ["SP_ME_BORDER"] = "1"
sp.me_search_sequence(fr, 352, 288, 16)
os.environ["SP_ME_BORDER"] = "0"
mark("sp.me_search_sequence (R = 16 plain order, 4 CTAs: both stages, byte-phase-0 tails)")
sp.me_search_sequence(fr, 352, 288, 16)
del os.environ["SP_ME_BORDER"]
mark("sp.jacobi1d_host (direct PCIe move-in)")
hd = torch.from_numpy(sp_inputs.jacobi_input(4099, seed=3)).pin_memory()
sp.Jacobi1DHost(4099, 150, 64, 0, direct_input=True).run(hd)
mark("sp.me_sad_search_range (flat range splitting a pair, R = 16 and 32)")
sp.me_sad_search_range(fr, 352, 288, 16, 7, 29)
sp.me_sad_search_range(fr3, 352, 288, 32, 3, 11)
mark("sp.me_sad_search_direct")
sp.me_sad_search_direct(fr2[:-1], fr2[1:], 130, 70, 8)
torch.cuda.synchronize()
print("sanitize target done")
