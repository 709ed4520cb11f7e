#!/bin/bash
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
for S in 4 8 12; do
VS_MODE=ready timeout 600 python bench.py --steps 3 --warmup 3 --no-e2e --no-cpu --slots $S --dump-log gpurun_out/b50_s$S.json > gpurun_out/b50_s$S.log 2>&1
done
