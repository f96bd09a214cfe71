"""bench.py's multi-GPU launch contract (CPU): `bench.py --gpus N` with no torchrun environment
runs itself under torch.distributed.run with one process per GPU and a 127.0.0.1 rendezvous,
forwarding its own arguments; under torchrun it insists on WORLD_SIZE == --gpus.  The N > 1
workload is BASELINE config 5 (J5, strong scaling) + the sharded M4 batch."""
import importlib.util
import os
import subprocess
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def _bench():
    spec = importlib.util.spec_from_file_location("bench_mod", os.path.join(ROOT, "bench.py"))
    m = importlib.util.module_from_spec(spec)
    spec.loader.exec_module(m)
    return m


def test_launch_cmd_is_torchrun_one_process_per_gpu():
    b = _bench()
    cmd = b.launch_cmd(["--gpus", "4", "--steps", "2"], 4, port=29555)
    assert cmd[:3] == [sys.executable, "-m", "torch.distributed.run"]
    assert "--nnodes=1" in cmd and "--nproc-per-node=4" in cmd
    assert "--master-addr=127.0.0.1" in cmd and "--master-port=29555" in cmd
    assert cmd[-4:] == ["--gpus", "4", "--steps", "2"] and cmd[-5].endswith("bench.py")


def test_world_size_must_match_gpus():
    env = dict(os.environ, WORLD_SIZE="1", RANK="0", LOCAL_RANK="0")
    out = subprocess.run([sys.executable, os.path.join(ROOT, "bench.py"), "--gpus", "2"], cwd=ROOT, env=env,
                         capture_output=True, text=True, timeout=120)
    assert out.returncode != 0 and "WORLD_SIZE=1" in (out.stderr + out.stdout)


def test_multi_gpu_workload_is_j5_strong_with_sharded_me():
    b = _bench()
    assert b.workload(1, 64)["name"] == "J3+M4" and b.workload(1, 64)["jac_n"] == 1 << 26
    w = b.workload(8, 64)
    assert w["name"] == "J5+M4" and w["jac_n"] == 1 << 30 and w["jac_t"] == 4096
    c = b.bench_config(4, 64)
    assert c["jacobi_global_n"] == 1 << 30 and "strong" in c["parallelism"] and c["me_pairs_global"] == 64
    # valid-candidate count of a sharded range sums to the batch's
    from paper_conf_ppopp_baskaranbkrrs08_b200 import partition
    rs = partition.me_row_ranges(64, 1080, 32, 8)
    assert sum(b.me_valid_sads(1920, 1080, 32, 64, r) for r in rs) == b.me_valid_sads(1920, 1080, 32, 64)
    assert b.me_valid_sads(1920, 1080, 32, 1) == 32_934_600
