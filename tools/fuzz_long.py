"""Long seeded fuzz of every Jacobi device entry point against the oracle (bit-exact), beyond
the GPU suite's 48 draws (development aid; profiles/r02_fuzz_long.txt):
    python tools/fuzz_long.py [cases] [first_seed]
Draws as tests/test_fuzz_gpu.py (n < 60,000, steps < 160, time tile incl. the bench's 128,
space tile, wavefront skew) and runs per-pass, persistent, wavefront-stream, host-buffer (the
in-place kernel's host-output instantiation at Tt >= 16) and cluster-resident calls."""
import sys
import time

import numpy as np
import torch

sys.path.insert(0, ".")
sys.path.insert(0, "tests")
import oracle  # noqa: E402
import paper_conf_ppopp_baskaranbkrrs08_b200 as sp  # noqa: E402
import sp_inputs  # noqa: E402


def bits(x):
    return np.ascontiguousarray(x).view(np.uint32)


def main():
    cases = int(sys.argv[1]) if len(sys.argv) > 1 else 300
    seed0 = int(sys.argv[2]) if len(sys.argv) > 2 else 5000
    rng = np.random.default_rng(seed0)
    fails, t0 = [], time.time()
    for c in range(cases):
        n = int(rng.integers(3, 60000))
        steps = int(rng.integers(0, 300))
        tt = int(rng.choice([1, 2, 3, 5, 8, 15, 16, 17, 31, 32, 33, 64, 96, 100, 127, 128]))
        H = sp.halo_of(tt)
        s_max = sp.jacobi1d_plan(1 << 20, 64, tt, 0)["space_tile"]
        S = 0 if rng.random() < 0.5 else min(s_max, int(rng.integers(1, max(2, s_max // 4 + 1))) * 4)
        a0 = sp_inputs.jacobi_input(n, seed=seed0 + c)
        want = bits(oracle.jacobi1d(a0, steps))
        case = (n, steps, tt, S)
        d = torch.from_numpy(a0.copy()).cuda()
        sp.jacobi1d_timetiled(d, steps, tt, S)
        if not np.array_equal(bits(d.cpu().numpy()), want):
            fails.append(("per-pass", case))
        d = torch.from_numpy(a0.copy()).cuda()
        sp.jacobi1d_timetiled_fused(d, steps, tt, S)
        if not np.array_equal(bits(d.cpu().numpy()), want):
            fails.append(("persistent", case))
        if steps > 0:
            reach = -(-H // (S if S else sp.jacobi1d_plan(n, steps, tt, 0)["space_tile"]))
            reach = max(reach, -(-H // (S if S else sp.jacobi1d_plan(n, steps, tt, 0)["persistent_space_tile"])))
            skew = 1
            while skew <= reach:
                skew *= 2
            skew *= int(rng.choice([1, 2, 8]))
            src = torch.from_numpy(a0.copy()).cuda()
            out = torch.empty_like(src)
            sp.jacobi1d_timetiled_stream(src, out, steps, tt, S, skew)
            if not np.array_equal(bits(out.cpu().numpy()), want):
                fails.append(("wavefront", case, skew))
        h = torch.from_numpy(a0.copy()).pin_memory()
        sp.Jacobi1DHost(n, steps, tt, S).run(h)
        torch.cuda.synchronize()
        if not np.array_equal(bits(h.numpy()), want):
            fails.append(("host", case))
        if n <= sp.jacobi1d_resident_capacity():
            src = torch.from_numpy(a0.copy()).cuda()
            out = sp.jacobi1d_resident(src, steps, out=torch.empty_like(src))
            if not np.array_equal(bits(out.cpu().numpy()), want):
                fails.append(("resident", case))
    print(f"{cases} cases (seed {seed0}), {len(fails)} failures, {time.time() - t0:.0f} s")
    for f in fails[:50]:
        print("FAIL", f)
    return 1 if fails else 0


if __name__ == "__main__":
    sys.exit(main())
