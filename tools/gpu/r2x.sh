set -x
O=gpurun_out/r2x_jac.txt
for rep in 1 2; do
for v in 14 15 16 17; do echo "== variant $v" >> $O; SP_JACOBI_VARIANT_FUSED=$v timeout 300 python tools/quick_time.py 56,64,72 --fused --no-me >> $O 2>&1; done
done
