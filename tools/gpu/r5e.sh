O=gpurun_out/r5e.txt
for rep in 1 2; do
echo "== packed tails, auto" >> $O; timeout 300 python tools/time_me_r16.py >> $O 2>&1
echo "== packed tails, SP_ME_BORDER=0" >> $O; SP_ME_BORDER=0 timeout 300 python tools/time_me_r16.py >> $O 2>&1
done
for v in "" 0 1; do echo "== dbg SP_ME_BORDER=$v" >> $O; SP_ME_BORDER=$v timeout 300 python tools/dbg_me16.py 64 >> $O 2>&1; done
timeout 1200 python -m pytest tests/test_me_gpu.py tests/test_me_shard_gpu.py tests/test_me_host_gpu.py -x -q > gpurun_out/r5e_pytest_me.txt 2>&1; echo rc=$? >> gpurun_out/r5e_pytest_me.txt
