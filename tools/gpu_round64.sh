#!/bin/bash
# step phases (inter-step gap) + bench variants
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 300 python tools/step_phases.py --steps 4 > gpurun_out/phases64.log 2>&1
B="timeout 400 python bench.py --steps 5 --warmup 3 --no-e2e --no-cpu"
$B > gpurun_out/b64_def.log 2>&1
VS_TCF_PAIR=0 $B > gpurun_out/b64_p0.log 2>&1
$B --slots 10 > gpurun_out/b64_s10.log 2>&1
$B --slots 14 > gpurun_out/b64_s14.log 2>&1
$B --group 6 > gpurun_out/b64_g6.log 2>&1
