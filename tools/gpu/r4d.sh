timeout 2400 python -m pytest tests -m gpu -x -q > gpurun_out/r4d_pytest_gpu.txt 2>&1; echo rc=$? >> gpurun_out/r4d_pytest_gpu.txt
for t in racecheck memcheck synccheck; do timeout 900 compute-sanitizer --tool $t python tools/sanitize_target.py > gpurun_out/r4d_san_$t.txt 2>&1; echo rc=$? >> gpurun_out/r4d_san_$t.txt; done
timeout 600 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/r4d_smoke.txt 2>&1; echo rc=$? >> gpurun_out/r4d_smoke.txt
O=gpurun_out/r4d.txt
echo "== fused, default routes" >> $O; timeout 300 python tools/quick_time.py 8,16,24,32,48,64,128 --fused --no-me >> $O 2>&1
timeout 1500 python tools/fuzz_long.py 1500 9000 > gpurun_out/r4d_fuzz.txt 2>&1; echo rc=$? >> gpurun_out/r4d_fuzz.txt
