#!/bin/bash
# queue depth 1 vs 2, interleaved, 3 repetitions of 10 steps
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
B="timeout 300 python bench.py --steps 10 --warmup 3 --no-e2e --no-cpu"
for rep in 1 2 3; do
  $B --qdepth 2 > gpurun_out/b92_q2_$rep.log 2>&1
  $B --qdepth 1 > gpurun_out/b92_q1_$rep.log 2>&1
done
