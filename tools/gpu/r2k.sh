set -x
SP_JACOBI_VARIANT=11 timeout 900 ncu --set full --clock-control none --import-source on -k regex:jacobi1d_pass_kernel -s 1 -c 1 -o gpurun_out/r2k_ip64 python tools/prof_target.py jacobi_fused 64 > gpurun_out/r2k_ncu.log 2>&1
O=gpurun_out/r2k_ip.txt
for v in 12 13; do echo "== variant $v" >> $O; SP_JACOBI_VARIANT=$v timeout 300 python tools/quick_time.py 48,64,80,96,128 --fused --no-me >> $O 2>&1; done
