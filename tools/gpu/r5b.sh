for v in "" 0 1; do echo "== SP_ME_BORDER=$v" >> gpurun_out/r5b.txt; SP_ME_BORDER=$v timeout 300 python tools/dbg_me16.py 24 >> gpurun_out/r5b.txt 2>&1; done
echo "== old lib" >> gpurun_out/r5b.txt; SP_LIB=tools/libsp_exp_old.so timeout 300 python tools/dbg_me16.py 24 >> gpurun_out/r5b.txt 2>&1
