#!/bin/bash
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 200 ./tools/probe_tc > gpurun_out/probe_tc.log 2>&1
timeout 900 python -m pytest tests/test_gpu_tiles.py tests/test_gpu_runtime.py -m gpu -q -p no:cacheprovider > gpurun_out/gpu_tests.log 2>&1
echo "tests exit $?" >> gpurun_out/gpu_tests.log
timeout 300 python tools/tilebench.py 1024 --streams 1 --types 0,4,3,2,1 --versions 1 > gpurun_out/tilebench.log 2>&1
timeout 300 python tools/tilebench.py 1024 --streams 4 --types 0,4,3,2,1 --versions 1 >> gpurun_out/tilebench.log 2>&1
timeout 300 ncu --set full --clock-control none --import-source on -k regex:tc_trsm -s 2 -c 1 -o gpurun_out/prof_trsm python tools/tilebench.py 1024 --types 2 --versions 1 > gpurun_out/ncu_trsm.log 2>&1
timeout 300 ncu --set full --clock-control none --import-source on -k regex:tc_gemm -s 5 -c 1 -o gpurun_out/prof_tc3 python tools/tilebench.py 1024 --types 0 --versions 1 > gpurun_out/ncu_tc.log 2>&1
timeout 600 python bench.py --steps 3 --warmup 3 --no-e2e --no-cpu --dump-log gpurun_out/bench_log.json --table-dump gpurun_out/table.txt > gpurun_out/bench_full.log 2>&1
