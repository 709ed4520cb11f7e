#!/bin/bash
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 600 python -m pytest tests/test_gpu_tiles.py tests/test_gpu_runtime.py tests/test_gpu_dist.py -q -p no:cacheprovider -x > gpurun_out/t48.log 2>&1; echo "exit $?" >> gpurun_out/t48.log
for i in 1 2; do
timeout 600 python bench.py --steps 3 --warmup 3 --no-e2e --no-cpu --slots 6 --dump-log gpurun_out/b48_$i.json > gpurun_out/b48_$i.log 2>&1
done
timeout 600 python bench.py --steps 3 --warmup 3 --no-e2e --no-cpu --slots 4 --dump-log gpurun_out/b48_s4.json > gpurun_out/b48_s4.log 2>&1
