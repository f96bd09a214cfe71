O=gpurun_out/r3p.txt
for rep in 1 2; do
for v in 20 23 24 25 26; do
echo "== variant $v" >> $O; SP_JACOBI_VARIANT_FUSED=$v timeout 300 python tools/quick_time.py 64,96,128 --fused --no-me >> $O 2>&1
done
done
