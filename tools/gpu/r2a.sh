set -x
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm --format=csv
timeout 900 python -m pytest tests/test_me_shard_gpu.py -x -q > gpurun_out/r2_shard.txt 2>&1; echo shard rc=$? >> gpurun_out/r2_shard.txt
for i in 1 2; do
timeout 300 python tools/quick_time.py 64 --fused > gpurun_out/r2_qt_acq$i.txt 2>&1
SP_LIB=tools/libsp_exp_noacq.so timeout 300 python tools/quick_time.py 64 --fused --no-me > gpurun_out/r2_qt_noacq$i.txt 2>&1
done
timeout 600 python bench.py --steps 10 --warmup 3 > gpurun_out/r2_bench1.txt 2>&1
timeout 1500 python -m pytest tests -m gpu -x -q > gpurun_out/r2_pytest_gpu.txt 2>&1; echo rc=$? >> gpurun_out/r2_pytest_gpu.txt
