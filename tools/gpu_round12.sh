#!/bin/bash
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_runtime.py tests/test_gpu_tiles.py -m gpu -q -p no:cacheprovider -x > gpurun_out/gpu_tests.log 2>&1
echo "tests exit $?" >> gpurun_out/gpu_tests.log
for cfg in "1 memops" "1 events" "0 memops"; do
  set -- $cfg
  VS_TRACKER=$2 VS_PRIORITY=$1 timeout 600 python bench.py --steps 3 --warmup 3 --no-e2e --no-cpu --dump-log gpurun_out/bench_log_$1_$2.json > gpurun_out/bench_$1_$2.log 2>&1
done
timeout 900 python bench.py --steps 3 --warmup 3 > gpurun_out/bench_default.log 2>&1
