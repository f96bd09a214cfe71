set -x
cd tools/microbench && nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o n2_calib n2_calib.cu -I ../../paper_conf_ppopp_baskaranbkrrs08_b200/csrc && ./n2_calib > ../../gpurun_out/r2_n2_calib2.json 2> ../../gpurun_out/r2_n2_calib2.err; cd ../..
timeout 300 python tools/time_small.py > gpurun_out/r2_latency.txt 2>&1
timeout 300 python tools/time_me_r16.py > gpurun_out/r2_me16.txt 2>&1
timeout 600 ncu --set full --clock-control none --import-source on -k regex:me_sad_kernel -s 1 -c 1 -o gpurun_out/r2_me16 python tools/prof_target.py me16 > gpurun_out/r2_me16_ncu.log 2>&1
