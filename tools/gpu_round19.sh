#!/bin/bash
# NN producer remap (4 rows x 128 B per LDG) + NEXT-4 bottom-level/queue-depth sweep
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 300 python -m pytest tests/test_gpu_tiles.py tests/test_gpu_runtime.py -q -p no:cacheprovider -x > gpurun_out/tiles.log 2>&1; echo "tiles exit $?" >> gpurun_out/tiles.log
timeout 300 python tools/tilebench.py 1024 --streams 1 --types 0,4 --versions 1 > gpurun_out/tilebench.log 2>&1
timeout 300 python tools/tilebench.py 1024 --streams 4 --types 0,4 --versions 1 >> gpurun_out/tilebench.log 2>&1
timeout 400 python bench.py --steps 3 --warmup 3 --dump-log gpurun_out/bench_log_default.json > gpurun_out/bench_default.log 2>&1
for cfg in "6 2 1" "6 1 0" "8 2 2" "6 2 3"; do
  set -- $cfg
  timeout 400 python bench.py --steps 3 --warmup 3 --slots $1 --priority $2 --qdepth $3 > gpurun_out/bench_s$1_p$2_q$3.log 2>&1
done
timeout 600 python -m pytest tests/test_gpu_fullsize.py -q -p no:cacheprovider -x > gpurun_out/fullsize.log 2>&1; echo "fullsize exit $?" >> gpurun_out/fullsize.log
