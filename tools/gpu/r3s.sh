timeout 2400 python -m pytest tests -m gpu -x -q > gpurun_out/r3s_pytest_gpu.txt 2>&1; echo rc=$? >> gpurun_out/r3s_pytest_gpu.txt
timeout 600 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/r3s_smoke.txt 2>&1; echo rc=$? >> gpurun_out/r3s_smoke.txt
for i in 1 2 3; do timeout 600 python bench.py > gpurun_out/r3s_bench$i.txt 2>&1; done
timeout 900 python bench.py --impl reference > gpurun_out/r3s_ref.txt 2>&1
SP_BENCH_SHARE_GPU=1 timeout 900 python bench.py --gpus 2 --steps 2 --warmup 3 > gpurun_out/r3s_share2.txt 2>&1; echo rc=$? >> gpurun_out/r3s_share2.txt
for tt in 64 128; do timeout 600 python tools/time_j5.py $tt >> gpurun_out/r3s_j5.txt 2>&1; done
timeout 300 python tools/time_small.py >> gpurun_out/r3s_small.txt 2>&1
