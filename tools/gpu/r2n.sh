set -x
timeout 900 ncu --set full --clock-control none --import-source on -k regex:jacobi1d_pass_kernel -s 1 -c 1 -o gpurun_out/r2n_ip64 python tools/prof_target.py jacobi_fused 64 > gpurun_out/r2n_ncu.log 2>&1
timeout 600 python bench.py > gpurun_out/r2n_bench.txt 2>&1
