O=gpurun_out/r5p.txt
echo "== current" >> $O; timeout 300 python tools/time_resident.py >> $O 2>&1
echo "== no Dirichlet restore (timing only)" >> $O; SP_LIB=tools/libsp_exp_nofix.so timeout 300 python tools/time_resident.py >> $O 2>&1
