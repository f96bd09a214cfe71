O=gpurun_out/r3q.txt
for rep in 1 2; do
for u in 2 1 4; do
L=""; [ $u != 2 ] && L=tools/libsp_exp_u$u.so
echo "== variant 20 unroll $u" >> $O; SP_LIB=$L timeout 300 python tools/quick_time.py 64,128 --fused --no-me >> $O 2>&1
done
done
timeout 2400 python -m pytest tests -m gpu -x -q > gpurun_out/r3q_pytest_gpu.txt 2>&1; echo rc=$? >> gpurun_out/r3q_pytest_gpu.txt
for t in racecheck memcheck synccheck; do timeout 900 compute-sanitizer --tool $t python tools/sanitize_target.py > gpurun_out/r3q_san_$t.txt 2>&1; echo rc=$? >> gpurun_out/r3q_san_$t.txt; done
