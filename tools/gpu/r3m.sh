set -x
./tools/microbench/tma_align > gpurun_out/r3m_tma_align.txt 2>&1; echo rc=$? >> gpurun_out/r3m_tma_align.txt
timeout 600 compute-sanitizer --tool memcheck ./tools/microbench/tma_align > gpurun_out/r3m_tma_align_san.txt 2>&1
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/r3m_launches_bench.csv python bench.py --steps 2 --warmup 3 --no-cpu-baseline > gpurun_out/r3m_bench_ncu.log 2>&1
