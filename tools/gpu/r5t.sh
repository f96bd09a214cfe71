# session-3 final validation and measurement
timeout 2700 python -m pytest tests -m gpu -x -q > gpurun_out/r5t_pytest_gpu.txt 2>&1; echo rc=$? >> gpurun_out/r5t_pytest_gpu.txt
timeout 600 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/r5t_smoke.txt 2>&1; echo rc=$? >> gpurun_out/r5t_smoke.txt
for i in 1 2 3; do timeout 600 python bench.py > gpurun_out/r5t_bench$i.txt 2>&1; done
timeout 900 python bench.py --impl reference > gpurun_out/r5t_ref.txt 2>&1
SP_BENCH_SHARE_GPU=1 timeout 900 python bench.py --gpus 2 --steps 2 --warmup 3 > gpurun_out/r5t_share2.txt 2>&1; echo rc=$? >> gpurun_out/r5t_share2.txt
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/r5t_launches_bench.csv python bench.py --steps 2 --warmup 3 --no-cpu-baseline > gpurun_out/r5t_bench_ncu.log 2>&1
timeout 300 python tools/time_small.py > gpurun_out/r5t_small.txt 2>&1
timeout 300 python tools/time_me_r16.py >> gpurun_out/r5t_small.txt 2>&1
