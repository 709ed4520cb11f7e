#!/bin/bash
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 600 python bench.py --steps 2 --warmup 3 --no-e2e --no-cpu --slots 6 --only ch --dump-log gpurun_out/b45_ch.json > gpurun_out/b45_ch.log 2>&1
