#!/bin/bash
# traced copy of libvsched.so (-DVS_PANEL_TRACE), installed over the package's library (GPU box only)
set -e
cd "${GRAFT_REPO_ROOT:-/root/repo}"
P=paper_conf_ipps_planasbal13_b200
mkdir -p scratch/tb
FL="-gencode arch=compute_100a,code=sm_100a -O3 -std=c++17 -lineinfo -Xcompiler -fPIC,-fvisibility=hidden -I include --expt-relaxed-constexpr -DVS_PANEL_TRACE"
objs=""
for f in $P/csrc/runtime/*.cpp; do o=scratch/tb/$(basename $f).o; /usr/local/cuda/bin/nvcc $FL -c $f -o $o & objs="$objs $o"; done
for f in $P/csrc/kernels/*.cu; do o=scratch/tb/$(basename $f).o; /usr/local/cuda/bin/nvcc $FL -x cu -c $f -o $o & objs="$objs $o"; done
wait
/usr/local/cuda/bin/nvcc -gencode arch=compute_100a,code=sm_100a -shared -o scratch/tb/libvsched.so $objs -cudart static -lpthread
cp scratch/tb/libvsched.so $P/libvsched.so   # NOTE: overwrites the in-tree library (delete it and rebuild afterwards)
