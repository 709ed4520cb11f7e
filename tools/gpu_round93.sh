#!/bin/bash
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 600 python -m pytest tests/test_gpu_fullsize.py tests/test_gpu_dist.py -q -p no:cacheprovider > gpurun_out/t93.log 2>&1; echo "exit $?" >> gpurun_out/t93.log
timeout 600 python bench.py > gpurun_out/b93.log 2>&1
