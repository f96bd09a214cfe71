O=gpurun_out/r6b.txt
for rep in 1 2; do
echo "== base (one warp per MB)" >> $O; timeout 300 python tools/time_small.py 2>&1 | grep M2 >> $O
echo "== SP_ME_R16_TY=4 (two warps per MB)" >> $O; SP_LIB=tools/libsp_exp_ty4.so timeout 300 python tools/time_small.py 2>&1 | grep M2 >> $O
done
SP_LIB=tools/libsp_exp_ty4.so timeout 300 python tools/time_me_r16.py >> $O 2>&1
