O=gpurun_out/r3v.txt
for rep in 1 2; do
echo "== per pass (staged 19)" >> $O; timeout 300 python tools/quick_time.py 4,8 --no-me >> $O 2>&1
echo "== persistent (staged 19 at Tt < 16)" >> $O; timeout 300 python tools/quick_time.py 4,8 --fused --no-me >> $O 2>&1
echo "== persistent (in place 20 forced)" >> $O; SP_JACOBI_VARIANT_FUSED=20 timeout 300 python tools/quick_time.py 4,8 --fused --no-me >> $O 2>&1
echo "== persistent (in place 16 forced)" >> $O; SP_JACOBI_VARIANT_FUSED=16 timeout 300 python tools/quick_time.py 4,8 --fused --no-me >> $O 2>&1
echo "== per pass (staged 5)" >> $O; SP_JACOBI_VARIANT=5 timeout 300 python tools/quick_time.py 4,8 --no-me >> $O 2>&1
done
