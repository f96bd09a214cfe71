set -x
timeout 900 ncu --set full --clock-control none --import-source on -k regex:jacobi1d_pass_kernel -s 1 -c 1 -o gpurun_out/r2r_jac python tools/prof_target.py jacobi_fused 64 > gpurun_out/r2r_ncu.log 2>&1
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/r2r_launches_bench.csv python bench.py --steps 2 --warmup 3 --no-cpu-baseline > gpurun_out/r2r_bench_ncu.log 2>&1
