set -x
timeout 1500 python -m pytest tests/test_jacobi_fused_gpu.py tests/test_jacobi_gpu.py tests/test_jacobi_stream_gpu.py tests/test_jacobi_stress_gpu.py tests/test_fuzz_gpu.py -x -q > gpurun_out/r2p_jac_tests.txt 2>&1; echo rc=$? >> gpurun_out/r2p_jac_tests.txt
timeout 900 compute-sanitizer --tool racecheck python tools/sanitize_target.py > gpurun_out/r2p_san_racecheck.txt 2>&1; echo rc=$? >> gpurun_out/r2p_san_racecheck.txt
timeout 900 compute-sanitizer --tool memcheck python tools/sanitize_target.py > gpurun_out/r2p_san_memcheck.txt 2>&1; echo rc=$? >> gpurun_out/r2p_san_memcheck.txt
timeout 300 python tools/quick_time.py 48,56,60,64,68,72,80,96 --fused --no-me > gpurun_out/r2p_tt.txt 2>&1
timeout 600 python bench.py > gpurun_out/r2p_bench.txt 2>&1
timeout 600 python bench.py > gpurun_out/r2p_bench2.txt 2>&1
timeout 300 python tools/time_j5.py > gpurun_out/r2p_j5.txt 2>&1
