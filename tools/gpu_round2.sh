#!/bin/bash
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
for v in 0 1 2 3; do timeout 30 ./tools/probe_mn_$v >> gpurun_out/probe_mn.log 2>&1; done
timeout 1200 python -m pytest tests -m gpu -q -p no:cacheprovider -x > gpurun_out/gpu_tests.log 2>&1
echo "tests exit $?" >> gpurun_out/gpu_tests.log
timeout 120 python __graft_entry__.py smoke > gpurun_out/smoke.log 2>&1
echo "smoke exit $?" >> gpurun_out/smoke.log
timeout 300 python bench.py --small --steps 3 --warmup 2 --no-cpu > gpurun_out/bench_small.log 2>&1
timeout 900 python bench.py --steps 3 --warmup 2 > gpurun_out/bench_full.log 2>&1
echo "bench exit $?" >> gpurun_out/bench_full.log
timeout 300 ncu --set full --clock-control none --import-source on -k regex:tc_gemm_kernel -s 3 -c 1 -o gpurun_out/prof_tc python tools/tilebench.py 1024 --types 4 --versions 1 > gpurun_out/ncu_tc.log 2>&1
