#!/bin/bash
# profiles: ncu full of oz_gemm (tilebench) and tcf_gemm (bench); launch list; default bench
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 600 ncu --set full --import-source on --clock-control none -k regex:oz_gemm -s 3 -c 1 -f -o gpurun_out/oz62 python tools/tilebench.py 2048 --types 0 --versions 6 --streams 1 --iters 3 > gpurun_out/ncu_oz62.log 2>&1; echo "exit $?" >> gpurun_out/ncu_oz62.log
timeout 900 ncu --set full --import-source on --clock-control none -k regex:tcf_gemm -s 3000 -c 1 -f -o gpurun_out/tcf62 python bench.py --steps 1 --warmup 1 --no-e2e --no-cpu > gpurun_out/ncu_tcf62.log 2>&1; echo "exit $?" >> gpurun_out/ncu_tcf62.log
timeout 1200 ncu --metrics gpu__time_duration.sum --clock-control none -c 9000 --csv --log-file gpurun_out/launches62.csv python bench.py --steps 1 --warmup 1 --no-e2e --no-cpu > gpurun_out/ncu_launch62.log 2>&1; echo "exit $?" >> gpurun_out/ncu_launch62.log
timeout 900 python bench.py --dump-log gpurun_out/b62.json > gpurun_out/b62.log 2>&1
