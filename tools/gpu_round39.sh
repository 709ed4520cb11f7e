#!/bin/bash
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
for S in 6 10 12; do
  timeout 600 python bench.py --steps 3 --warmup 3 --no-e2e --no-cpu --slots $S --dump-log gpurun_out/b39_s$S.json > gpurun_out/b39_s$S.log 2>&1
done
