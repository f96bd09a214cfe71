set -x
timeout 900 python -m pytest tests/test_peer_gpu.py tests/test_multidevice_gpu.py tests/test_me_shard_gpu.py -x -q > gpurun_out/r2q_peer_tests.txt 2>&1; echo rc=$? >> gpurun_out/r2q_peer_tests.txt
timeout 300 python tools/time_peer_single.py > gpurun_out/r2q_peer_single.txt 2>&1
SP_BENCH_SHARE_GPU=1 timeout 900 python bench.py --gpus 2 --steps 2 --warmup 3 > gpurun_out/r2q_bench_share2.txt 2>&1; echo rc=$? >> gpurun_out/r2q_bench_share2.txt
