#!/bin/bash
# first GPU validation pass
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
nvidia-smi > gpurun_out/smi.txt 2>&1
timeout 120 python -m pytest tests/test_gpu_tiles.py -x -q -k "test_matmul_tile and 128" > gpurun_out/t0.log 2>&1
echo "t0 exit $?" >> gpurun_out/t0.log
timeout 900 python -m pytest tests -m gpu -q -p no:cacheprovider > gpurun_out/gpu_tests.log 2>&1
echo "tests exit $?" >> gpurun_out/gpu_tests.log
timeout 120 python __graft_entry__.py smoke > gpurun_out/smoke.log 2>&1
echo "smoke exit $?" >> gpurun_out/smoke.log
timeout 300 python tools/tilebench.py 256 512 1024 > gpurun_out/tilebench.log 2>&1
timeout 300 python tools/tilebench.py 512 1024 --streams 4 --types 0,4 --versions 0,1 >> gpurun_out/tilebench.log 2>&1
echo "bench exit $?" >> gpurun_out/tilebench.log
