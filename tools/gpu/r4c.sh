O=gpurun_out/r4c.txt
for rep in 1 2; do
echo "== per pass (staged 19)" >> $O; timeout 300 python tools/quick_time.py 16,20,24,32,48 --no-me >> $O 2>&1
echo "== persistent (in place 20)" >> $O; SP_JACOBI_FUSED_PERSISTENT=1 timeout 300 python tools/quick_time.py 16,20,24,32,48 --fused --no-me >> $O 2>&1
echo "== persistent staged 19 forced" >> $O; SP_JACOBI_VARIANT_FUSED=19 timeout 300 python tools/quick_time.py 16,20,24,32,48 --fused --no-me >> $O 2>&1
done
