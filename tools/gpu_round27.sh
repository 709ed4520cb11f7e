#!/bin/bash
# tc_3xf16: tile parity, runtime forms, tile timing, bench
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 300 python -m pytest tests/test_gpu_tiles.py -q -p no:cacheprovider -x -k "3xf16 or row_scaling or integer or matmul_tile or gemm_nt" > gpurun_out/f16_tiles.log 2>&1; echo "exit $?" >> gpurun_out/f16_tiles.log
timeout 300 python -m pytest tests/test_gpu_runtime.py -q -p no:cacheprovider -x > gpurun_out/f16_runtime.log 2>&1; echo "exit $?" >> gpurun_out/f16_runtime.log
timeout 300 python tools/tilebench.py 1024 --streams 1 --types 0,4,3 --versions 1,5 > gpurun_out/f16_tilebench.log 2>&1
timeout 300 python tools/tilebench.py 1024 --streams 6 --types 0,4,3 --versions 1,5 >> gpurun_out/f16_tilebench.log 2>&1
timeout 600 python bench.py --dump-log gpurun_out/f16_bench_log.json > gpurun_out/f16_bench.log 2>&1; echo "exit $?" >> gpurun_out/f16_bench.log
