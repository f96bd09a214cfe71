timeout 900 ncu --set full --clock-control none --import-source on -k regex:jacobi1d_pass_kernel -s 2 -c 1 -o gpurun_out/r3w_pp8 python tools/prof_target.py jacobi 8 > gpurun_out/r3w_ncu.log 2>&1
timeout 900 ncu --set full --clock-control none --import-source on -k regex:me_sad_kernel -s 1 -c 1 -o gpurun_out/r3w_me16 python tools/prof_target.py me16 > gpurun_out/r3w_ncu16.log 2>&1
