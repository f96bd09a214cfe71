set -x
cd tools/microbench && nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o n2_calib n2_calib.cu -I ../../paper_conf_ppopp_baskaranbkrrs08_b200/csrc && ./n2_calib > ../../gpurun_out/r2_n2_calib.json 2> ../../gpurun_out/r2_n2_calib.err; cd ../..
timeout 900 python -m pytest tests/test_jacobi_gpu.py -k "loopback or J5" tests/test_me_shard_gpu.py -x -q > gpurun_out/r2_loopback.txt 2>&1; echo rc=$? >> gpurun_out/r2_loopback.txt
SP_BENCH_SHARE_GPU=1 timeout 900 python bench.py --gpus 2 --steps 2 --warmup 3 > gpurun_out/r2_bench_share2.txt 2>&1; echo rc=$? >> gpurun_out/r2_bench_share2.txt
timeout 600 python bench.py --steps 10 --warmup 3 > gpurun_out/r2_bench2.txt 2>&1
