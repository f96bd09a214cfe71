set -x
O=gpurun_out/r3j.txt
for rep in 1 2; do
for v in 16 17 18; do echo "== variant $v unroll 2" >> $O; SP_JACOBI_VARIANT_FUSED=$v timeout 300 python tools/quick_time.py 56,64,72 --fused --no-me >> $O 2>&1; done
for u in 1 4; do echo "== variant 16 unroll $u" >> $O; SP_LIB=tools/libsp_exp_u$u.so timeout 300 python tools/quick_time.py 64 --fused --no-me >> $O 2>&1; done
echo "== variant 17 unroll 4" >> $O; SP_JACOBI_VARIANT_FUSED=17 SP_LIB=tools/libsp_exp_u4.so timeout 300 python tools/quick_time.py 64 --fused --no-me >> $O 2>&1
done
