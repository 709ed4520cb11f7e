#!/bin/bash
# final knob sweep (two repetitions each): qdepth, group size, slots
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
B="timeout 300 python bench.py --steps 5 --warmup 3 --no-e2e --no-cpu"
for rep in 1 2; do
  $B > gpurun_out/b91_def_$rep.log 2>&1
  $B --qdepth 3 > gpurun_out/b91_q3_$rep.log 2>&1
  $B --qdepth 1 > gpurun_out/b91_q1_$rep.log 2>&1
  $B --group 12 > gpurun_out/b91_g12_$rep.log 2>&1
  $B --slots 10 > gpurun_out/b91_s10_$rep.log 2>&1
done
