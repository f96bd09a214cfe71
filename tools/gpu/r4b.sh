O=gpurun_out/r4b.txt
echo "== fused at Tt 4 / 8 (default route: per pass below 16)" >> $O; timeout 300 python tools/quick_time.py 4,8,16 --fused --no-me >> $O 2>&1
echo "== fused at Tt 4 / 8, SP_JACOBI_FUSED_PERSISTENT=1" >> $O; SP_JACOBI_FUSED_PERSISTENT=1 timeout 300 python tools/quick_time.py 4,8 --fused --no-me >> $O 2>&1
timeout 1800 python -m pytest tests/test_jacobi_fused_gpu.py tests/test_fuzz_gpu.py tests/test_jacobi_stress_gpu.py tests/test_jacobi_gpu.py tests/test_multidevice_gpu.py -x -q > gpurun_out/r4b_pytest.txt 2>&1; echo rc=$? >> gpurun_out/r4b_pytest.txt
timeout 600 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/r4b_smoke.txt 2>&1; echo rc=$? >> gpurun_out/r4b_smoke.txt
