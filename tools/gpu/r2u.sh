set -x
timeout 2400 python -m pytest tests -m gpu -x -q > gpurun_out/r2u_pytest_gpu.txt 2>&1; echo rc=$? >> gpurun_out/r2u_pytest_gpu.txt
timeout 600 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/r2u_smoke.txt 2>&1; echo rc=$? >> gpurun_out/r2u_smoke.txt
for i in 1 2 3; do timeout 600 python bench.py > gpurun_out/r2u_bench$i.txt 2>&1; done
timeout 900 python bench.py --impl reference --steps 2 --warmup 3 > gpurun_out/r2u_ref.txt 2>&1
timeout 300 python tools/time_small.py > gpurun_out/r2u_latency.txt 2>&1
timeout 300 python tools/time_me_r16.py > gpurun_out/r2u_me16.txt 2>&1
timeout 300 python tools/time_j5.py > gpurun_out/r2u_j5.txt 2>&1
