timeout 1200 python -m pytest tests/test_me_host_gpu.py tests/test_jacobi_stream_gpu.py -x -q -k "host or cif or 1080p or device_outputs or rejects" > gpurun_out/r5w_pytest.txt 2>&1; echo rc=$? >> gpurun_out/r5w_pytest.txt
O=gpurun_out/r5w.txt
for rep in 1 2 3; do timeout 300 python tools/time_me_e2e.py >> $O 2>&1; done
