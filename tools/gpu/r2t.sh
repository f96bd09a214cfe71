set -x
timeout 900 python -m pytest tests/test_me_gpu.py tests/test_me_shard_gpu.py -x -q > gpurun_out/r2t_me_tests.txt 2>&1; echo rc=$? >> gpurun_out/r2t_me_tests.txt
O=gpurun_out/r2t_me.txt
for rep in 1 2; do
echo "== s11 (product)" >> $O; timeout 300 python tools/quick_time.py --me-only >> $O 2>&1
echo "== s00" >> $O; SP_LIB=tools/libsp_exp_s00.so timeout 300 python tools/quick_time.py --me-only >> $O 2>&1
echo "== s10" >> $O; SP_LIB=tools/libsp_exp_s10.so timeout 300 python tools/quick_time.py --me-only >> $O 2>&1
echo "== s01" >> $O; SP_LIB=tools/libsp_exp_s01.so timeout 300 python tools/quick_time.py --me-only >> $O 2>&1
done
