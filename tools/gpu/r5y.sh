for i in 1 2 3; do timeout 600 python bench.py > gpurun_out/r5y_bench$i.txt 2>&1; done
timeout 2700 python -m pytest tests -m gpu -x -q > gpurun_out/r5y_pytest_gpu.txt 2>&1; echo rc=$? >> gpurun_out/r5y_pytest_gpu.txt
timeout 600 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/r5y_smoke.txt 2>&1; echo rc=$? >> gpurun_out/r5y_smoke.txt
