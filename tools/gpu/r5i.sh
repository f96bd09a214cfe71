O=gpurun_out/r5i.txt
for sh in small tiny mid large; do SP_JACOBI_RESIDENT=$sh timeout 300 python tools/time_resident.py >> $O 2>&1; done
SP_LIB=tools/libsp_exp_old.so SP_JACOBI_RESIDENT=small timeout 300 python tools/time_resident.py 2>&1 | sed 's/^/OLD /' >> $O
timeout 900 python -m pytest tests/test_jacobi_resident_gpu.py -x -q > gpurun_out/r5i_pytest.txt 2>&1; echo rc=$? >> gpurun_out/r5i_pytest.txt
for sh in tiny mid; do SP_JACOBI_RESIDENT=$sh timeout 900 python -m pytest tests/test_jacobi_resident_gpu.py -x -q -k "not capacity" 2>&1 | tail -2 | sed "s/^/$sh /" >> gpurun_out/r5i_pytest.txt; done
