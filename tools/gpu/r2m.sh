set -x
timeout 1500 python -m pytest tests/test_jacobi_fused_gpu.py tests/test_jacobi_gpu.py tests/test_jacobi_stream_gpu.py tests/test_jacobi_stress_gpu.py tests/test_fuzz_gpu.py tests/test_jacobi_resident_gpu.py tests/test_peer_gpu.py -x -q > gpurun_out/r2m_jac_tests.txt 2>&1; echo rc=$? >> gpurun_out/r2m_jac_tests.txt
for t in racecheck memcheck synccheck; do timeout 900 compute-sanitizer --tool $t python tools/sanitize_target.py > gpurun_out/r2m_san_$t.txt 2>&1; echo rc=$? >> gpurun_out/r2m_san_$t.txt; done
timeout 600 python bench.py > gpurun_out/r2m_bench.txt 2>&1
timeout 300 python tools/quick_time.py 56,64,72,80,96 --fused --no-me > gpurun_out/r2m_tt.txt 2>&1
