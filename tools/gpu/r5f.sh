O=gpurun_out/r5f.txt
timeout 1200 python -m pytest tests/test_me_gpu.py tests/test_me_shard_gpu.py tests/test_me_host_gpu.py -x -q > gpurun_out/r5f_pytest_me.txt 2>&1; echo rc=$? >> gpurun_out/r5f_pytest_me.txt
for rep in 1 2; do
echo "== M4 class order (auto)" >> $O; timeout 300 python tools/quick_time.py --me-only >> $O 2>&1
echo "== M4 SP_ME_BORDER=0" >> $O; SP_ME_BORDER=0 timeout 300 python tools/quick_time.py --me-only >> $O 2>&1
echo "== r16 auto" >> $O; timeout 300 python tools/time_me_r16.py >> $O 2>&1
done
