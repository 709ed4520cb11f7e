#!/bin/bash
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 600 python -m pytest tests -m gpu -q -p no:cacheprovider -x > gpurun_out/t49.log 2>&1; echo "exit $?" >> gpurun_out/t49.log
timeout 300 python __graft_entry__.py smoke > gpurun_out/smoke49.log 2>&1; echo "exit $?" >> gpurun_out/smoke49.log
timeout 900 python bench.py --dump-log gpurun_out/b49.json > gpurun_out/b49.log 2>&1
timeout 1500 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/launches49.csv python bench.py --steps 1 --warmup 1 --no-e2e --no-cpu > gpurun_out/ncu_launch49.log 2>&1; echo "exit $?" >> gpurun_out/ncu_launch49.log
timeout 900 ncu --set full --import-source on --clock-control none -k regex:tcf_gemm -s 400 -c 1 -f -o gpurun_out/tcf_bench python bench.py --steps 1 --warmup 1 --no-e2e --no-cpu > gpurun_out/ncu_full49.log 2>&1; echo "exit $?" >> gpurun_out/ncu_full49.log
