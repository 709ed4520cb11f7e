#!/bin/bash
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 600 python -m pytest tests/test_gpu_runtime.py tests/test_gpu_dist.py -q -p no:cacheprovider -x > gpurun_out/rt44.log 2>&1; echo "exit $?" >> gpurun_out/rt44.log
timeout 600 python bench.py --steps 3 --warmup 3 --no-e2e --no-cpu --slots 6 --only ch --dump-log gpurun_out/b44_ch.json > gpurun_out/b44_ch.log 2>&1
timeout 600 python bench.py --steps 3 --warmup 3 --no-e2e --no-cpu --slots 4 --dump-log gpurun_out/b44_s4.json > gpurun_out/b44_s4.log 2>&1
timeout 600 python bench.py --steps 3 --warmup 3 --no-e2e --no-cpu --slots 6 --dump-log gpurun_out/b44_s6.json > gpurun_out/b44_s6.log 2>&1
