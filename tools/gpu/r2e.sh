set -x
O=gpurun_out/r2e_jac.txt
for rep in 1 2; do
for st in 0 3000 6000; do echo "== stagger $st" >> $O; SP_JACOBI_STAGGER=$st timeout 200 python tools/quick_time.py 64 --fused --no-me >> $O 2>&1; done
echo "== grab2" >> $O; SP_LIB=tools/libsp_exp_grab2.so timeout 200 python tools/quick_time.py 64 --fused --no-me >> $O 2>&1
echo "== grab2 stagger 3000" >> $O; SP_JACOBI_STAGGER=3000 SP_LIB=tools/libsp_exp_grab2.so timeout 200 python tools/quick_time.py 64 --fused --no-me >> $O 2>&1
done
SP_LIB=tools/libsp_exp_grab2.so timeout 900 python -m pytest tests/test_jacobi_fused_gpu.py tests/test_jacobi_stream_gpu.py -x -q > gpurun_out/r2e_grab2_tests.txt 2>&1; echo rc=$? >> gpurun_out/r2e_grab2_tests.txt
