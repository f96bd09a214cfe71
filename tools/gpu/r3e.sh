set -x
timeout 1200 python tools/n1_ablation.py > gpurun_out/r3e_n1.jsonl 2> gpurun_out/r3e_n1.err
timeout 900 python -m pytest tests/test_me_gpu.py -k prepared tests/test_jacobi_resident_gpu.py -x -q > gpurun_out/r3e_tests.txt 2>&1; echo rc=$? >> gpurun_out/r3e_tests.txt
