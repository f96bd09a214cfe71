set -x
O=gpurun_out/r2l_ip.txt
for rep in 1 2; do
for v in 11 12; do
echo "== variant $v unroll 1" >> $O; SP_JACOBI_VARIANT=$v timeout 300 python tools/quick_time.py 64,96,128 --fused --no-me >> $O 2>&1
echo "== variant $v unroll 2" >> $O; SP_LIB=tools/libsp_exp_u2.so SP_JACOBI_VARIANT=$v timeout 300 python tools/quick_time.py 64,96,128 --fused --no-me >> $O 2>&1
echo "== variant $v unroll 4" >> $O; SP_LIB=tools/libsp_exp_u4.so SP_JACOBI_VARIANT=$v timeout 300 python tools/quick_time.py 64,96,128 --fused --no-me >> $O 2>&1
done
done
