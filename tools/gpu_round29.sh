#!/bin/bash
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 600 ncu --set full --import-source on --clock-control none -k regex:tcf_gemm_kernel -s 3 -c 1 -f -o gpurun_out/tcf1 python tools/tilebench.py 1024 --streams 1 --types 4 --versions 5 --iters 2 > gpurun_out/ncu_tcf1.log 2>&1
