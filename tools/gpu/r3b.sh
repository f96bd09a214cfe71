set -x
O=gpurun_out/r3b_timing.txt
for rep in 1 2; do
echo "== product" >> $O; timeout 300 python tools/quick_time.py 64 --fused --no-me >> $O 2>&1
for t in 8 11; do echo "== timing $t" >> $O; SP_LIB=tools/libsp_exp_t$t.so timeout 300 python tools/quick_time.py 64 --fused --no-me >> $O 2>&1; done
done
