# round 2 session 3: R = 16 class order with half-frame border searches
timeout 900 python -m pytest tests/test_me_gpu.py tests/test_me_shard_gpu.py tests/test_me_host_gpu.py -x -q > gpurun_out/r5a_pytest_me.txt 2>&1; echo rc=$? >> gpurun_out/r5a_pytest_me.txt
O=gpurun_out/r5a.txt
for rep in 1 2; do
echo "== new, auto" >> $O; timeout 300 python tools/time_me_r16.py >> $O 2>&1
echo "== new, SP_ME_BORDER=0" >> $O; SP_ME_BORDER=0 timeout 300 python tools/time_me_r16.py >> $O 2>&1
echo "== old lib" >> $O; SP_LIB=tools/libsp_exp_old.so timeout 300 python tools/time_me_r16.py >> $O 2>&1
echo "== M4 new" >> $O; timeout 300 python tools/quick_time.py --me-only >> $O 2>&1
echo "== M4 old" >> $O; SP_LIB=tools/libsp_exp_old.so timeout 300 python tools/quick_time.py --me-only >> $O 2>&1
done
echo "== latency" >> $O; timeout 300 python tools/time_small.py >> $O 2>&1
