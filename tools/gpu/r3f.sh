set -x
timeout 1500 python -m pytest tests/test_jacobi_fused_gpu.py tests/test_jacobi_gpu.py tests/test_jacobi_stream_gpu.py tests/test_fuzz_gpu.py tests/test_peer_gpu.py tests/test_jacobi_stress_gpu.py -x -q > gpurun_out/r3f_tests.txt 2>&1; echo rc=$? >> gpurun_out/r3f_tests.txt
timeout 300 python tools/quick_time.py 4,8,16,32,64 --fused --no-me > gpurun_out/r3f_tt.txt 2>&1
