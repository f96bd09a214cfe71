O=gpurun_out/r3x.txt
for rep in 1 2; do
for v in 19 20 16 14; do
echo "== per pass, variant $v" >> $O; SP_JACOBI_VARIANT=$v timeout 300 python tools/quick_time.py 4,8,16 --no-me >> $O 2>&1
done
done
