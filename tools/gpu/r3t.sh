O=gpurun_out/r3t.txt
for rep in 1 2; do
echo "== old: staged variant 19, skew 512" >> $O; SP_JACOBI_VARIANT_FUSED=19 timeout 300 python tools/time_stream.py --tt=64,128 --skews=0 --host >> $O 2>&1
for sk in 128 256 512 1024; do
echo "== new: in place K = 56 with staged host move-out, skew $sk" >> $O; SP_JACOBI_SKEW=$sk timeout 300 python tools/time_stream.py --tt=64,128 --skews=0 --host >> $O 2>&1
done
done
echo "== device J3" >> $O; timeout 300 python tools/quick_time.py 64,128 --fused --no-me >> $O 2>&1
timeout 1800 python -m pytest tests/test_jacobi_stream_gpu.py tests/test_jacobi_fused_gpu.py tests/test_fuzz_gpu.py tests/test_jacobi_stress_gpu.py -x -q > gpurun_out/r3t_pytest.txt 2>&1; echo rc=$? >> gpurun_out/r3t_pytest.txt
