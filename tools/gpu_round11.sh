#!/bin/bash
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 1500 python -m pytest tests -m gpu -q -p no:cacheprovider > gpurun_out/gpu_tests.log 2>&1
echo "tests exit $?" >> gpurun_out/gpu_tests.log
for cfg in "0 0 memops" "0 0 events" "0 1 memops" "8 1 memops" "16 1 memops" "32 1 memops"; do
  set -- $cfg
  VS_TRACKER=$3 VS_LOOKAHEAD=$1 VS_PRIORITY=$2 timeout 600 python bench.py --steps 3 --warmup 3 --no-e2e --no-cpu --dump-log gpurun_out/bench_log_$1_$2_$3.json > gpurun_out/bench_$1_$2_$3.log 2>&1
done
