"""ncu target: the cluster-resident Jacobi at N = 8192, T = 4096 (development aid)."""
import sys
import torch
sys.path.insert(0, ".")
import paper_conf_ppopp_baskaranbkrrs08_b200 as sp  # noqa: E402
import sp_inputs  # noqa: E402
n = int(sys.argv[1]) if len(sys.argv) > 1 else 8192
a = torch.from_numpy(sp_inputs.jacobi_input(n, seed=1)).cuda()
sp.jacobi1d_resident(a, 4096)
torch.cuda.synchronize()
print("done")
