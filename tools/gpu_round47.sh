#!/bin/bash
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 600 python -m pytest tests/test_gpu_tiles.py tests/test_gpu_runtime.py -q -p no:cacheprovider -x > gpurun_out/t47.log 2>&1; echo "exit $?" >> gpurun_out/t47.log
timeout 300 python tools/tilebench.py 1024 --streams 1 --types 2 --versions 1,5 > gpurun_out/tb47.log 2>&1
timeout 600 python bench.py --steps 2 --warmup 3 --no-e2e --no-cpu --slots 6 --only ch --dump-log gpurun_out/b47_ch.json > gpurun_out/b47_ch.log 2>&1
timeout 600 python bench.py --steps 2 --warmup 3 --no-e2e --no-cpu --slots 6 --dump-log gpurun_out/b47_both.json > gpurun_out/b47_both.log 2>&1
