#!/bin/bash
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
for LA in 0 48 96; do
VS_LOOKAHEAD=$LA timeout 600 python bench.py --steps 2 --warmup 3 --no-e2e --no-cpu --slots 6 --only ch --dump-log gpurun_out/b46_ch_$LA.json > gpurun_out/b46_ch_$LA.log 2>&1
VS_LOOKAHEAD=$LA timeout 600 python bench.py --steps 2 --warmup 3 --no-e2e --no-cpu --slots 6 --dump-log gpurun_out/b46_both_$LA.json > gpurun_out/b46_both_$LA.log 2>&1
done
