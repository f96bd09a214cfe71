# session-3 final bench lines + final R = 16 capture (CSV exported on the box)
for i in 1 2 3; do timeout 600 python bench.py > gpurun_out/r5v_bench$i.txt 2>&1; done
mkdir -p /tmp/r5v
timeout 900 ncu --set full --clock-control none --import-source on -k regex:me_sad_kernel -s 1 -c 1 -o /tmp/r5v/me16 python tools/prof_target.py me16 > gpurun_out/r5v_ncu16.log 2>&1
ncu -i /tmp/r5v/me16.ncu-rep --page raw --csv > gpurun_out/r5v_me16_raw.csv 2>&1
ncu -i /tmp/r5v/me16.ncu-rep --page source --csv --print-source sass > gpurun_out/r5v_me16_src.csv 2>&1
