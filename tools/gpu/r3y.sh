O=gpurun_out/r3y.txt
for rep in 1 2 3; do
echo "== phase build on FMA (new)" >> $O; timeout 300 python tools/time_me_r16.py >> $O 2>&1; timeout 300 python tools/quick_time.py --me-only >> $O 2>&1
echo "== phase build SHF (old)" >> $O; SP_LIB=tools/libsp_exp_shf.so timeout 300 python tools/time_me_r16.py >> $O 2>&1; SP_LIB=tools/libsp_exp_shf.so timeout 300 python tools/quick_time.py --me-only >> $O 2>&1
done
timeout 1800 python -m pytest tests -m gpu -x -q -k "me or ME" > gpurun_out/r3y_pytest.txt 2>&1; echo rc=$? >> gpurun_out/r3y_pytest.txt
