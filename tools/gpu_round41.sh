#!/bin/bash
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 600 python -m pytest tests/test_gpu_runtime.py tests/test_gpu_dist.py -q -p no:cacheprovider -x > gpurun_out/rt41.log 2>&1; echo "exit $?" >> gpurun_out/rt41.log
for S in 6 10; do
timeout 600 python bench.py --steps 3 --warmup 3 --no-e2e --no-cpu --slots $S --dump-log gpurun_out/b41_s$S.json > gpurun_out/b41_s$S.log 2>&1
done
