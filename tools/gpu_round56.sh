#!/bin/bash
# launch-cost probe; hold / slots sweep
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
nvcc -gencode arch=compute_100a,code=sm_100a -O2 -o /tmp/probe_launch tools/probe_launch.cu && /tmp/probe_launch > gpurun_out/probe_launch.log 2>&1
B="timeout 400 python bench.py --steps 5 --warmup 3 --no-e2e --no-cpu"
export VS_GROUP_HOLD=1
for cfg in "100 12" "200 12" "60 16" "100 16" "400 12"; do
  set -- $cfg
  VS_GROUP_US=$1 $B --slots $2 > gpurun_out/b56_h$1s$2.log 2>&1
done
VS_GROUP_US=100 $B --slots 12 --group 16 > gpurun_out/b56_h100s12g16.log 2>&1
