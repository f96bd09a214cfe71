O=gpurun_out/r5d.txt
for rep in 1 2; do
echo "== new (noinline)" >> $O; timeout 300 python tools/time_me_r16.py >> $O 2>&1
echo "== inlined border search" >> $O; SP_LIB=tools/libsp_exp_binl.so timeout 300 python tools/time_me_r16.py >> $O 2>&1
done
SP_LIB=tools/libsp_exp_binl.so SP_ME_BORDER=1 timeout 300 python tools/dbg_me16.py 32 >> $O 2>&1
timeout 900 ncu --set full --clock-control none --import-source on -k regex:me_sad_kernel -s 1 -c 1 -o gpurun_out/r5d_me16 python tools/prof_target.py me16 > gpurun_out/r5d_ncu16.log 2>&1
