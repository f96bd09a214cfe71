set -x
O=gpurun_out/r2s_acq.txt
for rep in 1 2 3; do
echo "== acq" >> $O; timeout 300 python tools/quick_time.py 64 --fused --no-me >> $O 2>&1
echo "== noacq" >> $O; SP_LIB=tools/libsp_exp_noacq.so timeout 300 python tools/quick_time.py 64 --fused --no-me >> $O 2>&1
done
