timeout 900 python -m pytest tests/test_jacobi_stream_gpu.py -x -q > gpurun_out/r5k_pytest.txt 2>&1; echo rc=$? >> gpurun_out/r5k_pytest.txt
O=gpurun_out/r5k.txt
for rep in 1 2; do timeout 600 python tools/time_host_decomp.py 512 >> $O 2>&1; done
