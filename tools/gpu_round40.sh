#!/bin/bash
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 600 python bench.py --steps 3 --warmup 3 --no-e2e --no-cpu --slots 10 --dump-log gpurun_out/b40_both.json > gpurun_out/b40_both.log 2>&1
timeout 600 python bench.py --steps 3 --warmup 3 --no-e2e --no-cpu --slots 10 --only mm --dump-log gpurun_out/b40_mm.json > gpurun_out/b40_mm.log 2>&1
VS_TRACKER=memops timeout 600 python bench.py --steps 3 --warmup 3 --no-e2e --no-cpu --slots 10 --dump-log gpurun_out/b40_memops.json > gpurun_out/b40_memops.log 2>&1
