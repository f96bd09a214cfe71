set -x
timeout 300 python tools/time_me_r16.py > gpurun_out/r2d_me16.txt 2>&1
timeout 300 python tools/time_me_r16.py >> gpurun_out/r2d_me16.txt 2>&1
timeout 300 python tools/quick_time.py --me-only >> gpurun_out/r2d_me16.txt 2>&1
timeout 900 python -m pytest tests/test_me_gpu.py tests/test_me_stress_gpu.py tests/test_me_shard_gpu.py tests/test_me_host_gpu.py tests/test_fuzz_gpu.py -x -q > gpurun_out/r2d_me_tests.txt 2>&1; echo rc=$? >> gpurun_out/r2d_me_tests.txt
for t in racecheck memcheck synccheck; do timeout 900 compute-sanitizer --tool $t python tools/sanitize_target.py > gpurun_out/r2d_san_$t.txt 2>&1; echo rc=$? >> gpurun_out/r2d_san_$t.txt; done
timeout 600 ncu --set full --clock-control none --import-source on -k regex:me_sad_kernel -s 1 -c 1 -o gpurun_out/r2d_me16 python tools/prof_target.py me16 > gpurun_out/r2d_me16_ncu.log 2>&1
