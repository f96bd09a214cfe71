#!/bin/bash
# Experimental libsp variant that recompiles only jacobi.cu with extra defines (development aid):
#   tools/build_jac_exp.sh NAME -DFOO=1 ...  ->  tools/libsp_exp_NAME.so  (other objects from build/libsp)
set -e
name=$1; shift
cd "$(dirname "$0")/.."
mkdir -p build/exp_jac_$name
nvcc -gencode arch=compute_100a,code=sm_100a -O3 -lineinfo -std=c++17 -I include -Xcompiler -fPIC,-O2,-ffp-contract=off \
  --fmad=false "$@" -c paper_conf_ppopp_baskaranbkrrs08_b200/csrc/jacobi.cu -o build/exp_jac_$name/jacobi.cu.o 2>/dev/null
nvcc -gencode arch=compute_100a,code=sm_100a -shared -o tools/libsp_exp_$name.so build/libsp/api.cpp.o \
  build/libsp/planner.cpp.o build/libsp/comm.cpp.o build/exp_jac_$name/jacobi.cu.o build/libsp/me.cu.o \
  build/libsp/ablation.cu.o build/libsp/exec.cu.o -cudart static -ldl -lpthread
echo tools/libsp_exp_$name.so
