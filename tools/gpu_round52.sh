#!/bin/bash
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
VS_MODE=ready timeout 600 python bench.py --steps 3 --warmup 3 --no-e2e --no-cpu --slots 8 --qdepth 2 --dump-log gpurun_out/b52_ready.json > gpurun_out/b52_ready.log 2>&1
timeout 600 python bench.py --steps 3 --warmup 3 --no-e2e --no-cpu --slots 4 --dump-log gpurun_out/b52_ra.json > gpurun_out/b52_ra.log 2>&1
timeout 600 python bench.py --steps 3 --warmup 3 --no-e2e --no-cpu --slots 8 --dump-log gpurun_out/b52_ra8.json > gpurun_out/b52_ra8.log 2>&1
