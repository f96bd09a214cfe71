#!/bin/bash
# Jacobi kernel geometry sweep: variants x time tiles at J3 (N = 2^26, T = 1024)
for v in 0 1 2 3 4; do
  echo "== variant $v"
  SP_JACOBI_VARIANT=$v python tools/quick_time.py ${1:-16,24,32} --no-me 2>&1 | sed 's/plan=.*space_tile/space_tile/'
done
