"""ncu target: one cluster-resident Jacobi call (N = 4,096, T = 4,096; development aid)."""
import sys

import torch

sys.path.insert(0, ".")
import paper_conf_ppopp_baskaranbkrrs08_b200 as sp  # noqa: E402
import sp_inputs  # noqa: E402

x = torch.from_numpy(sp_inputs.jacobi_input(4096)).cuda()
y = torch.empty_like(x)
for _ in range(2):
    sp.jacobi1d_resident(x, 4096, out=y)
torch.cuda.synchronize()
