set -x
timeout 2400 python -m pytest tests -m gpu -x -q > gpurun_out/r3l_pytest_gpu.txt 2>&1; echo rc=$? >> gpurun_out/r3l_pytest_gpu.txt
for t in racecheck memcheck synccheck; do timeout 900 compute-sanitizer --tool $t python tools/sanitize_target.py > gpurun_out/r3l_san_$t.txt 2>&1; echo rc=$? >> gpurun_out/r3l_san_$t.txt; done
timeout 600 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/r3l_smoke.txt 2>&1; echo rc=$? >> gpurun_out/r3l_smoke.txt
for i in 1 2 3; do timeout 600 python bench.py > gpurun_out/r3l_bench$i.txt 2>&1; done
SP_BENCH_SHARE_GPU=1 timeout 900 python bench.py --gpus 2 --steps 2 --warmup 3 > gpurun_out/r3l_share2.txt 2>&1; echo rc=$? >> gpurun_out/r3l_share2.txt
