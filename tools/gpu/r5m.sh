timeout 2700 python -m pytest tests -m gpu -x -q > gpurun_out/r5m_pytest_gpu.txt 2>&1; echo rc=$? >> gpurun_out/r5m_pytest_gpu.txt
timeout 600 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/r5m_smoke.txt 2>&1; echo rc=$? >> gpurun_out/r5m_smoke.txt
for t in racecheck memcheck synccheck; do timeout 900 compute-sanitizer --tool $t python tools/sanitize_target.py > gpurun_out/r5m_san_$t.txt 2>&1; echo rc=$? >> gpurun_out/r5m_san_$t.txt; done
for i in 1 2; do timeout 600 python bench.py > gpurun_out/r5m_bench$i.txt 2>&1; done
