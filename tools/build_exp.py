"""Build an experimental libsp variant with extra nvcc defines (development aid):
    python tools/build_exp.py NAME -DFOO=1 ...   ->  tools/libsp_exp_NAME.so
Run it with SP_LIB=tools/libsp_exp_NAME.so (the binding loads that file instead)."""
import os
import subprocess
import sys

sys.path.insert(0, os.path.join(os.path.dirname(os.path.abspath(__file__)), "..", "paper_conf_ppopp_baskaranbkrrs08_b200"))
import _build as B  # noqa: E402

name, defs = sys.argv[1], sys.argv[2:]
out_dir = os.path.join(B.ROOT, "build", "exp_" + name)
os.makedirs(out_dir, exist_ok=True)
inc = os.path.join(B.ROOT, "include")
objs = []
for src in B.SOURCES:
    obj = os.path.join(out_dir, src + ".o")
    cmd = [B.nvcc(), *B.ARCH, "-O3", "-lineinfo", "-std=c++17", "-I", inc, "-Xcompiler", "-fPIC,-O2,-ffp-contract=off",
           *defs, "-c", os.path.join(B.CSRC, src), "-o", obj]
    cmd += ["--fmad=false"] if src.endswith(".cu") else []
    if not src.endswith(".cu"):
        cmd[1:1] = ["-x", "c++"]
    subprocess.check_call(cmd)
    objs.append(obj)
lib = os.path.join(B.ROOT, "tools", f"libsp_exp_{name}.so")
subprocess.check_call([B.nvcc(), *B.ARCH, "-shared", "-o", lib, *objs, "-cudart", "static", "-ldl", "-lpthread"])
print(lib)
