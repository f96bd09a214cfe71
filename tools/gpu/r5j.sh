timeout 600 python tools/time_host_decomp.py 256,512,1024 > gpurun_out/r5j.txt 2>&1
