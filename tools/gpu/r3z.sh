timeout 2700 python -m pytest tests -m gpu -x -q > gpurun_out/r3z_pytest_gpu.txt 2>&1; echo rc=$? >> gpurun_out/r3z_pytest_gpu.txt
timeout 600 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/r3z_smoke.txt 2>&1; echo rc=$? >> gpurun_out/r3z_smoke.txt
for t in racecheck memcheck synccheck; do timeout 900 compute-sanitizer --tool $t python tools/sanitize_target.py > gpurun_out/r3z_san_$t.txt 2>&1; echo rc=$? >> gpurun_out/r3z_san_$t.txt; done
for i in 1 2 3; do timeout 600 python bench.py > gpurun_out/r3z_bench$i.txt 2>&1; done
timeout 900 python bench.py --impl reference > gpurun_out/r3z_ref.txt 2>&1
SP_BENCH_SHARE_GPU=1 timeout 900 python bench.py --gpus 2 --steps 2 --warmup 3 > gpurun_out/r3z_share2.txt 2>&1; echo rc=$? >> gpurun_out/r3z_share2.txt
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/r3z_launches_bench.csv python bench.py --steps 2 --warmup 3 --no-cpu-baseline > gpurun_out/r3z_bench_ncu.log 2>&1
timeout 300 python tools/time_small.py > gpurun_out/r3z_small.txt 2>&1
