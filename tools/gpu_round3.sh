#!/bin/bash
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 60 ./tools/probe_tc > gpurun_out/probe_tc.log 2>&1
timeout 900 python -m pytest tests/test_gpu_tiles.py tests/test_gpu_runtime.py -m gpu -q -p no:cacheprovider > gpurun_out/gpu_tests.log 2>&1
echo "tests exit $?" >> gpurun_out/gpu_tests.log
