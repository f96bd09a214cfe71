O=gpurun_out/r5n.txt
for rep in 1 2; do
echo "== new (launch first)" >> $O; timeout 300 python tools/time_me_e2e.py >> $O 2>&1
echo "== old (copies enqueued first)" >> $O; SP_LIB=tools/libsp_exp_old.so timeout 300 python tools/time_me_e2e.py >> $O 2>&1
done
timeout 900 python -m pytest tests/test_me_host_gpu.py -x -q > gpurun_out/r5n_pytest.txt 2>&1; echo rc=$? >> gpurun_out/r5n_pytest.txt
