#!/bin/bash
# ncu full captures of the tc GEMM kernel, NN (matmul) and NT (gemm_nt), b=1024
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 600 ncu --set full --import-source on --clock-control none -k regex:tc_gemm_kernel -c 1 -f -o gpurun_out/gemm_nn python tools/tilebench.py 1024 --streams 1 --types 0 --versions 1 --iters 1 > gpurun_out/ncu_gemm_nn.log 2>&1
timeout 600 ncu --set full --import-source on --clock-control none -k regex:tc_gemm_kernel -c 1 -f -o gpurun_out/gemm_nt python tools/tilebench.py 1024 --streams 1 --types 4 --versions 1 --iters 1 > gpurun_out/ncu_gemm_nt.log 2>&1
