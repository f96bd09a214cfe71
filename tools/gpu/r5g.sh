O=gpurun_out/r5g.txt
for rep in 1 2 3; do
for lib in r16only binl; do
echo "== M4 $lib auto" >> $O; SP_LIB=tools/libsp_exp_$lib.so timeout 300 python tools/quick_time.py --me-only >> $O 2>&1
done
echo "== M4 binl SP_ME_BORDER=0" >> $O; SP_ME_BORDER=0 SP_LIB=tools/libsp_exp_binl.so timeout 300 python tools/quick_time.py --me-only >> $O 2>&1
done
echo "== r16 binl" >> $O; SP_LIB=tools/libsp_exp_binl.so timeout 300 python tools/time_me_r16.py >> $O 2>&1
echo "== r16 binl" >> $O; SP_LIB=tools/libsp_exp_binl.so timeout 300 python tools/time_me_r16.py >> $O 2>&1
