timeout 1200 python -m pytest tests/test_jacobi_stream_gpu.py tests/test_me_host_gpu.py -x -q > gpurun_out/r5u_pytest.txt 2>&1; echo rc=$? >> gpurun_out/r5u_pytest.txt
O=gpurun_out/r5u.txt
for rep in 1 2; do timeout 300 python tools/time_host_e2e.py 128 >> $O 2>&1; timeout 300 python tools/time_me_e2e.py >> $O 2>&1; done
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/r5u_launches_bench.csv python bench.py --steps 2 --warmup 3 --no-cpu-baseline > gpurun_out/r5u_bench_ncu.log 2>&1; echo rc=$? >> gpurun_out/r5u_bench_ncu.log
