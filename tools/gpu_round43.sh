#!/bin/bash
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
for S in 4 6 8; do
timeout 600 python bench.py --steps 3 --warmup 3 --no-e2e --no-cpu --slots $S --group 8 --dump-log gpurun_out/b43_s$S.json > gpurun_out/b43_s$S.log 2>&1
done
timeout 600 python bench.py --steps 3 --warmup 3 --no-e2e --no-cpu --slots 6 --group 8 --only mm --dump-log gpurun_out/b43_mm.json > gpurun_out/b43_mm.log 2>&1
timeout 600 python bench.py --steps 3 --warmup 3 --no-e2e --no-cpu --slots 6 --group 8 --only ch --dump-log gpurun_out/b43_ch.json > gpurun_out/b43_ch.log 2>&1
