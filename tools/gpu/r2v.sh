set -x
timeout 900 ncu --set full --clock-control none --import-source on -k regex:me_sad_kernel -s 1 -c 1 -o gpurun_out/r2v_me python tools/prof_target.py me > gpurun_out/r2v_ncu.log 2>&1
