O=gpurun_out/r5o.txt
for rep in 1 2; do
echo "== launch first" >> $O; timeout 300 python tools/time_me_e2e.py >> $O 2>&1
echo "== + ready cache" >> $O; SP_LIB=tools/libsp_exp_rdy.so timeout 300 python tools/time_me_e2e.py >> $O 2>&1
done
SP_LIB=tools/libsp_exp_rdy.so timeout 900 python -m pytest tests/test_me_host_gpu.py -x -q > gpurun_out/r5o_pytest.txt 2>&1; echo rc=$? >> gpurun_out/r5o_pytest.txt
