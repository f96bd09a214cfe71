timeout 1500 python -m pytest tests/test_fuzz_gpu.py -x -q -k multi_wave > gpurun_out/r5x_pytest.txt 2>&1; echo rc=$? >> gpurun_out/r5x_pytest.txt
