O=gpurun_out/r5r.txt
echo "== select restore" >> $O; timeout 300 python tools/time_resident.py >> $O 2>&1
echo "== jump-table restore (A/B build)" >> $O; SP_LIB=tools/libsp_exp_jump.so timeout 300 python tools/time_resident.py >> $O 2>&1
echo "== select restore, large shape" >> $O; SP_JACOBI_RESIDENT=large timeout 300 python tools/time_resident.py >> $O 2>&1
timeout 900 python -m pytest tests/test_jacobi_resident_gpu.py tests/test_fuzz_gpu.py -x -q > gpurun_out/r5r_pytest.txt 2>&1; echo rc=$? >> gpurun_out/r5r_pytest.txt
SP_JACOBI_RESIDENT=large timeout 900 python -m pytest tests/test_jacobi_resident_gpu.py -x -q -k "not capacity" >> gpurun_out/r5r_pytest.txt 2>&1; echo rc=$? >> gpurun_out/r5r_pytest.txt
