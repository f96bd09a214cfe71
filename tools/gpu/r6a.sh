timeout 1500 python tools/fuzz_long.py 1500 9100 > gpurun_out/r6a_fuzz.txt 2>&1; echo rc=$? >> gpurun_out/r6a_fuzz.txt
