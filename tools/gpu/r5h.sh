O=gpurun_out/r5h.txt
for rep in 1 2 3; do
echo "== r16 HEAD" >> $O; timeout 300 python tools/time_me_r16.py >> $O 2>&1
echo "== r16 fin1" >> $O; SP_LIB=tools/libsp_exp_fin1.so timeout 300 python tools/time_me_r16.py >> $O 2>&1
done
echo "== M4 fin1" >> $O; SP_LIB=tools/libsp_exp_fin1.so timeout 300 python tools/quick_time.py --me-only >> $O 2>&1
SP_LIB=tools/libsp_exp_fin1.so timeout 300 python tools/dbg_me16.py 64 >> $O 2>&1
SP_LIB=tools/libsp_exp_fin1.so SP_ME_BORDER=0 timeout 300 python tools/dbg_me16.py 64 >> $O 2>&1
