O=gpurun_out/r3u.txt
for rep in 1 2; do
echo "== device J3 (plain instantiation)" >> $O; timeout 300 python tools/quick_time.py 64,128 --fused --no-me >> $O 2>&1
echo "== host path, in place K = 56, host-out instantiation, skew 512" >> $O; timeout 300 python tools/time_stream.py --tt=64,128 --skews=0 --host >> $O 2>&1
done
timeout 1800 python -m pytest tests/test_jacobi_stream_gpu.py tests/test_jacobi_fused_gpu.py tests/test_fuzz_gpu.py tests/test_jacobi_stress_gpu.py tests/test_jacobi_gpu.py -x -q > gpurun_out/r3u_pytest.txt 2>&1; echo rc=$? >> gpurun_out/r3u_pytest.txt
for t in racecheck memcheck synccheck; do timeout 900 compute-sanitizer --tool $t python tools/sanitize_target.py > gpurun_out/r3u_san_$t.txt 2>&1; echo rc=$? >> gpurun_out/r3u_san_$t.txt; done
timeout 600 python bench.py > gpurun_out/r3u_bench.txt 2>&1
