set -x
timeout 1800 python -m pytest tests -m gpu -x -q > gpurun_out/r2i_pytest_gpu.txt 2>&1; echo rc=$? >> gpurun_out/r2i_pytest_gpu.txt
timeout 600 python bench.py > gpurun_out/r2i_bench.txt 2>&1
timeout 600 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/r2i_smoke.txt 2>&1; echo rc=$? >> gpurun_out/r2i_smoke.txt
timeout 300 python tools/time_me_r16.py > gpurun_out/r2i_me16.txt 2>&1
