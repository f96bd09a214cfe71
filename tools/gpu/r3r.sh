for i in 1 2 3; do timeout 600 python bench.py > gpurun_out/r3r_bench$i.txt 2>&1; done
SP_BENCH_SHARE_GPU=1 timeout 900 python bench.py --gpus 2 --steps 2 --warmup 3 > gpurun_out/r3r_share2.txt 2>&1; echo rc=$? >> gpurun_out/r3r_share2.txt
timeout 600 python bench.py --time-tile 64 > gpurun_out/r3r_bench_tt64.txt 2>&1
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/r3r_launches_bench.csv python bench.py --steps 2 --warmup 3 --no-cpu-baseline > gpurun_out/r3r_bench_ncu.log 2>&1
timeout 900 ncu --set full --clock-control none --import-source on -k regex:jacobi1d_pass_kernel -s 1 -c 1 -o gpurun_out/r3r_jac python tools/prof_target.py jacobi_fused 128 > gpurun_out/r3r_ncu.log 2>&1
