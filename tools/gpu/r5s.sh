O=gpurun_out/r5s.txt
echo "== select restore (small shape only)" >> $O; timeout 300 python tools/time_resident.py >> $O 2>&1
echo "== large shape (jump table)" >> $O; SP_JACOBI_RESIDENT=large timeout 300 python tools/time_resident.py >> $O 2>&1
timeout 300 python tools/time_small.py >> $O 2>&1
timeout 900 python -m pytest tests/test_jacobi_resident_gpu.py tests/test_fuzz_gpu.py -x -q > gpurun_out/r5s_pytest.txt 2>&1; echo rc=$? >> gpurun_out/r5s_pytest.txt
SP_JACOBI_RESIDENT=large timeout 900 python -m pytest tests/test_jacobi_resident_gpu.py -x -q -k "not capacity" >> gpurun_out/r5s_pytest.txt 2>&1; echo rc=$? >> gpurun_out/r5s_pytest.txt
SP_JACOBI_RESIDENT=small timeout 900 python -m pytest tests/test_jacobi_resident_gpu.py -x -q -k "not capacity" >> gpurun_out/r5s_pytest.txt 2>&1; echo rc=$? >> gpurun_out/r5s_pytest.txt
