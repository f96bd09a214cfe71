set -x
O=gpurun_out/r2z_host.txt
echo "== staged (default host path)" >> $O; timeout 300 python tools/time_stream.py --tt=64 --skews=0 --host >> $O 2>&1
for sk in 256 512 1024; do
echo "== in place (variant 14) skew $sk" >> $O; SP_JACOBI_VARIANT=14 SP_JACOBI_SKEW=$sk timeout 300 python tools/time_stream.py --tt=64 --skews=0 --host >> $O 2>&1
done
echo "== staged skew 256" >> $O; SP_JACOBI_SKEW=256 timeout 300 python tools/time_stream.py --tt=64 --skews=0 --host >> $O 2>&1
