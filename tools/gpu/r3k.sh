set -x
O=gpurun_out/r3k.txt
for rep in 1 2; do
for v in 5 19; do
echo "== staged variant $v: host path" >> $O; SP_JACOBI_VARIANT=$v SP_JACOBI_VARIANT_FUSED=16 timeout 300 python tools/time_stream.py --tt=64 --skews=0 --host >> $O 2>&1
echo "== staged variant $v: per pass Tt 8 / 64" >> $O; SP_JACOBI_VARIANT=$v SP_JACOBI_VARIANT_FUSED=16 timeout 300 python tools/quick_time.py 8,64 --no-me >> $O 2>&1
done
done
