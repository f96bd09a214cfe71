set -x
O=gpurun_out/r3c.txt
for rep in 1 2 3; do
echo "== new (predicated move-out)" >> $O; timeout 300 python tools/quick_time.py 64 --fused --no-me >> $O 2>&1
echo "== old" >> $O; SP_LIB=tools/libsp_exp_old.so timeout 300 python tools/quick_time.py 64 --fused --no-me >> $O 2>&1
done
