timeout 1500 python tools/fuzz_long.py 400 5000 > gpurun_out/r4a_fuzz.txt 2>&1; echo rc=$? >> gpurun_out/r4a_fuzz.txt
timeout 900 python -m pytest tests/test_fuzz_gpu.py -q > gpurun_out/r4a_fuzz_suite.txt 2>&1; echo rc=$? >> gpurun_out/r4a_fuzz_suite.txt
