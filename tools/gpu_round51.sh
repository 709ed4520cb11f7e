#!/bin/bash
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
for S in 4 8; do for Q in 1 2 4; do
VS_MODE=ready timeout 600 python bench.py --steps 3 --warmup 3 --no-e2e --no-cpu --slots $S --qdepth $Q --dump-log gpurun_out/b51_s${S}_q$Q.json > gpurun_out/b51_s${S}_q$Q.log 2>&1
done; done
