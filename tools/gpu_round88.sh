#!/bin/bash
# oz GEMM with precomputed slice descriptors: tests + tilebench
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 300 python -m pytest tests/test_gpu_tiles.py -q -p no:cacheprovider -k "oz or 6" > gpurun_out/t88.log 2>&1; echo "exit $?" >> gpurun_out/t88.log
timeout 300 python tools/tilebench.py 1024 2048 --types 0,4,3 --versions 6 --streams 1 > gpurun_out/tb88.log 2>&1
timeout 300 python tools/tilebench.py 2048 --types 0 --versions 6 --streams 8 >> gpurun_out/tb88.log 2>&1
