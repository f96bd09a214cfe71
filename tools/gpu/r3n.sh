for a in "0 0" "0 16" "0 5" "0 8" "0 -3" "0 1" "16 0" "32 0" "48 0" "96 0" "32 16" "32 5"; do ./tools/microbench/tma_align $a; done > gpurun_out/r3n_tma_align.txt 2>&1
