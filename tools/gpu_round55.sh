#!/bin/bash
# A/B: sized kernel-parameter blocks (default), idle-flush hold of pending groups; cfg5 rerun
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
B="timeout 400 python bench.py --steps 5 --warmup 3 --no-e2e --no-cpu"
$B --dump-log gpurun_out/b55_def.json > gpurun_out/b55_def.log 2>&1
VS_GROUP_HOLD=1 $B --dump-log gpurun_out/b55_h20.json > gpurun_out/b55_h20.log 2>&1
VS_GROUP_HOLD=1 VS_GROUP_US=60 $B > gpurun_out/b55_h60.log 2>&1
VS_GROUP_HOLD=1 VS_GROUP_US=60 $B --slots 12 > gpurun_out/b55_h60s12.log 2>&1
timeout 900 python tools/sweep_cfg5.py --out gpurun_out/cfg5.json > gpurun_out/cfg5.log 2>&1; echo "exit $?" >> gpurun_out/cfg5.log
