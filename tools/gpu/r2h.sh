set -x
O=gpurun_out/r2h_time.txt
for rep in 1 2; do
echo "== product" >> $O; timeout 300 python tools/time_me_r16.py >> $O 2>&1
echo "== noborder" >> $O; SP_LIB=tools/libsp_exp_noborder.so timeout 300 python tools/time_me_r16.py >> $O 2>&1
echo "== borderinl" >> $O; SP_LIB=tools/libsp_exp_borderinl.so timeout 300 python tools/time_me_r16.py >> $O 2>&1
done
timeout 600 ncu --set full --clock-control none --import-source on -k regex:me_sad_kernel -s 1 -c 1 -o gpurun_out/r2h_me16 python tools/prof_target.py me16 > gpurun_out/r2h_me16_ncu.log 2>&1
timeout 900 python -m pytest tests/test_me_gpu.py -x -q > gpurun_out/r2h_me_tests.txt 2>&1; echo rc=$? >> gpurun_out/r2h_me_tests.txt
