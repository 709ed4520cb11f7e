#!/bin/bash
# parts of the step alone: matmul only, Cholesky only (critical path), with logs
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 400 python bench.py --steps 5 --warmup 3 --no-e2e --no-cpu --only ch --dump-log gpurun_out/b69_ch.json > gpurun_out/b69_ch.log 2>&1
timeout 400 python bench.py --steps 5 --warmup 3 --no-e2e --no-cpu --only mm --dump-log gpurun_out/b69_mm.json > gpurun_out/b69_mm.log 2>&1
timeout 300 python tools/tilebench.py 1024 --types 1,2 --versions 1,5 --streams 1 > gpurun_out/tb69.log 2>&1
