mkdir -p /tmp/r5q
for v in cur nofix; do
  if [ $v = nofix ]; then export SP_LIB=tools/libsp_exp_nofix.so; fi
  timeout 600 ncu --set full --clock-control none --import-source on -k regex:cluster_kernel -s 1 -c 1 -o /tmp/r5q/$v python tools/prof_resident.py > gpurun_out/r5q_ncu_$v.log 2>&1
  ncu -i /tmp/r5q/$v.ncu-rep --page raw --csv > gpurun_out/r5q_${v}_raw.csv 2>&1
  ncu -i /tmp/r5q/$v.ncu-rep --page source --csv --print-source sass > gpurun_out/r5q_${v}_src.csv 2>&1
done
ls -la gpurun_out/
