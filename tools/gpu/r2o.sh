set -x
O=gpurun_out/r2o_ip.txt
for rep in 1 2; do
for v in 11 14; do
echo "== variant $v unroll 2" >> $O; SP_JACOBI_VARIANT_FUSED=$v timeout 300 python tools/quick_time.py 64,72 --fused --no-me >> $O 2>&1
done
echo "== variant 14 unroll 1" >> $O; SP_LIB=tools/libsp_exp_u1.so SP_JACOBI_VARIANT_FUSED=14 timeout 300 python tools/quick_time.py 64,72 --fused --no-me >> $O 2>&1
echo "== variant 14 unroll 4" >> $O; SP_LIB=tools/libsp_exp_u4.so SP_JACOBI_VARIANT_FUSED=14 timeout 300 python tools/quick_time.py 64,72 --fused --no-me >> $O 2>&1
done
