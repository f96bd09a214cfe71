set -x
timeout 900 python -m pytest tests/test_me_gpu.py tests/test_me_shard_gpu.py tests/test_me_host_gpu.py -x -q > gpurun_out/r2y_me_tests.txt 2>&1; echo rc=$? >> gpurun_out/r2y_me_tests.txt
O=gpurun_out/r2y_me.txt
for rep in 1 2; do
echo "== fastdiv" >> $O; timeout 300 python tools/time_me_r16.py >> $O 2>&1; timeout 300 python tools/quick_time.py --me-only >> $O 2>&1
echo "== old" >> $O; SP_LIB=tools/libsp_exp_old.so timeout 300 python tools/time_me_r16.py >> $O 2>&1; SP_LIB=tools/libsp_exp_old.so timeout 300 python tools/quick_time.py --me-only >> $O 2>&1
done
