set -x
timeout 900 python -m pytest tests/test_me_gpu.py tests/test_me_stress_gpu.py tests/test_me_shard_gpu.py tests/test_me_host_gpu.py tests/test_fuzz_gpu.py -x -q > gpurun_out/r3d_me_tests.txt 2>&1; echo rc=$? >> gpurun_out/r3d_me_tests.txt
O=gpurun_out/r3d.txt
for rep in 1 2; do
echo "== ty4 (2 warps)" >> $O; timeout 300 python tools/time_me_r16.py >> $O 2>&1
echo "== ty8 (1 warp)" >> $O; SP_LIB=tools/libsp_exp_ty8.so timeout 300 python tools/time_me_r16.py >> $O 2>&1
done
timeout 300 python tools/time_small.py > gpurun_out/r3d_latency.txt 2>&1
