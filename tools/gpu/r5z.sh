O=gpurun_out/r5z.txt
for rep in 1 2; do
echo "== M4 base" >> $O; timeout 300 python tools/quick_time.py --me-only >> $O 2>&1
echo "== M4 allow-expensive-optimizations" >> $O; SP_LIB=tools/libsp_exp_aeo.so timeout 300 python tools/quick_time.py --me-only >> $O 2>&1
echo "== r16 base" >> $O; timeout 300 python tools/time_me_r16.py >> $O 2>&1
echo "== r16 aeo" >> $O; SP_LIB=tools/libsp_exp_aeo.so timeout 300 python tools/time_me_r16.py >> $O 2>&1
done
