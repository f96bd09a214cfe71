set -x
timeout 600 python -m pytest tests/test_multidevice_gpu.py -x -q > gpurun_out/r2f_multidev.txt 2>&1; echo rc=$? >> gpurun_out/r2f_multidev.txt
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/r2f_launches_bench.csv python bench.py --steps 2 --warmup 3 --no-cpu-baseline > gpurun_out/r2f_bench_ncu.log 2>&1
timeout 900 ncu --set full --clock-control none --import-source on -k regex:jacobi1d_pass_kernel -s 1 -c 1 -o gpurun_out/r2f_jac python tools/prof_target.py jacobi_fused > gpurun_out/r2f_jac_ncu.log 2>&1
timeout 900 ncu --set full --clock-control none --import-source on -k regex:me_sad_kernel -s 1 -c 1 -o gpurun_out/r2f_me python tools/prof_target.py me > gpurun_out/r2f_me_ncu.log 2>&1
