#!/bin/bash
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 120 ./tools/probe_tcf 1024 16 > gpurun_out/probe_tcf.log 2>&1
timeout 300 python -m pytest tests/test_gpu_tiles.py -q -p no:cacheprovider -x -k "3xf16 or row_scaling or integer or matmul_tile or gemm_nt" > gpurun_out/f16_tiles.log 2>&1; echo "exit $?" >> gpurun_out/f16_tiles.log
timeout 300 python -m pytest tests/test_gpu_runtime.py -q -p no:cacheprovider -x -k 3xf16 > gpurun_out/f16_runtime.log 2>&1; echo "exit $?" >> gpurun_out/f16_runtime.log
