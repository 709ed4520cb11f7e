#!/bin/bash
# GEMM changes: parity + tile timing + bench
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 300 python -m pytest tests/test_gpu_tiles.py tests/test_gpu_runtime.py -q -p no:cacheprovider -x > gpurun_out/tiles_all.log 2>&1; echo "tiles_all exit $?" >> gpurun_out/tiles_all.log
timeout 300 python tools/tilebench.py 1024 --streams 1 --types 0,4,3 --versions 1 > gpurun_out/tilebench_gemm.log 2>&1
timeout 300 python tools/tilebench.py 1024 --streams 4 --types 0,4,3 --versions 1 >> gpurun_out/tilebench_gemm.log 2>&1
timeout 400 python bench.py --steps 3 --warmup 3 --dump-log gpurun_out/bench_log_default.json > gpurun_out/bench_default.log 2>&1
