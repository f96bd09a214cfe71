set -x
timeout 900 python -m pytest tests/test_me_gpu.py -x -q > gpurun_out/r2g_me_tests.txt 2>&1; echo rc=$? >> gpurun_out/r2g_me_tests.txt
timeout 300 python tools/time_me_r16.py > gpurun_out/r2g_time.txt 2>&1
timeout 300 python tools/quick_time.py --me-only >> gpurun_out/r2g_time.txt 2>&1
timeout 300 python tools/time_me_r16.py >> gpurun_out/r2g_time.txt 2>&1
timeout 300 python tools/quick_time.py --me-only >> gpurun_out/r2g_time.txt 2>&1
timeout 900 python -m pytest tests/test_me_stress_gpu.py tests/test_me_shard_gpu.py tests/test_me_host_gpu.py tests/test_fuzz_gpu.py tests/test_ablation_gpu.py -x -q > gpurun_out/r2g_me_tests2.txt 2>&1; echo rc=$? >> gpurun_out/r2g_me_tests2.txt
timeout 900 compute-sanitizer --tool racecheck python tools/sanitize_target.py > gpurun_out/r2g_san_racecheck.txt 2>&1; echo rc=$? >> gpurun_out/r2g_san_racecheck.txt
timeout 900 compute-sanitizer --tool memcheck python tools/sanitize_target.py > gpurun_out/r2g_san_memcheck.txt 2>&1; echo rc=$? >> gpurun_out/r2g_san_memcheck.txt
