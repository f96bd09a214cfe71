set -x
O=gpurun_out/r2j_ip.txt
SP_JACOBI_VARIANT=11 timeout 900 python -m pytest tests/test_jacobi_fused_gpu.py tests/test_jacobi_gpu.py tests/test_jacobi_stream_gpu.py -x -q -k "not peer" > gpurun_out/r2j_ip_tests.txt 2>&1; echo rc=$? >> gpurun_out/r2j_ip_tests.txt
for v in 5 11; do echo "== variant $v" >> $O; SP_JACOBI_VARIANT=$v timeout 300 python tools/quick_time.py 32,48,64,80,96,128 --fused --no-me >> $O 2>&1; done
echo "== variant 11 again" >> $O; SP_JACOBI_VARIANT=11 timeout 300 python tools/quick_time.py 64,96 --fused --no-me >> $O 2>&1
