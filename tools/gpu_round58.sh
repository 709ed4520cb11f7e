#!/bin/bash
# completion ring: runtime tests + bench
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 600 python -m pytest tests/test_gpu_runtime.py tests/test_gpu_cfg5.py tests/test_gpu_dist.py -q -p no:cacheprovider -x > gpurun_out/t58.log 2>&1; echo "exit $?" >> gpurun_out/t58.log
timeout 600 python bench.py --no-e2e --no-cpu --dump-log gpurun_out/b58.json > gpurun_out/b58.log 2>&1
timeout 600 python bench.py --no-e2e --no-cpu --slots 8 > gpurun_out/b58_s8.log 2>&1
timeout 600 python bench.py --no-e2e --no-cpu --slots 16 > gpurun_out/b58_s16.log 2>&1
