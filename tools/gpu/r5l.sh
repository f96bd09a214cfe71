O=gpurun_out/r5l.txt
for D in 128 256 512 1024; do SP_JACOBI_SKEW=$D timeout 600 python tools/time_host_e2e.py 64,128 >> $O 2>&1; done
