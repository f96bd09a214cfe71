set -x
timeout 1500 python -m pytest tests/test_jacobi_fused_gpu.py tests/test_jacobi_gpu.py tests/test_jacobi_stream_gpu.py tests/test_fuzz_gpu.py tests/test_peer_gpu.py tests/test_jacobi_stress_gpu.py tests/test_multidevice_gpu.py -x -q > gpurun_out/r3i_tests.txt 2>&1; echo rc=$? >> gpurun_out/r3i_tests.txt
timeout 900 compute-sanitizer --tool racecheck python tools/sanitize_target.py > gpurun_out/r3i_san_racecheck.txt 2>&1; echo rc=$? >> gpurun_out/r3i_san_racecheck.txt
timeout 900 compute-sanitizer --tool memcheck python tools/sanitize_target.py > gpurun_out/r3i_san_memcheck.txt 2>&1; echo rc=$? >> gpurun_out/r3i_san_memcheck.txt
timeout 300 python tools/quick_time.py 32,64 --fused --no-me > gpurun_out/r3i_tt.txt 2>&1
timeout 300 python tools/time_j5.py > gpurun_out/r3i_j5.txt 2>&1
timeout 300 python tools/time_peer_single.py > gpurun_out/r3i_peer_single.txt 2>&1
