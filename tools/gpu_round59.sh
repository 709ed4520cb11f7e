#!/bin/bash
# CTA-pair (A multicast) tcf GEMM: tile tests, runtime tests, tilebench and bench A/B
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 300 python -m pytest tests/test_gpu_tiles.py -q -p no:cacheprovider -x > gpurun_out/t59_tiles.log 2>&1; echo "exit $?" >> gpurun_out/t59_tiles.log
timeout 300 python -m pytest tests/test_gpu_runtime.py -q -p no:cacheprovider -x > gpurun_out/t59_rt.log 2>&1; echo "exit $?" >> gpurun_out/t59_rt.log
for p in 0 1; do
  VS_TCF_PAIR=$p timeout 300 python tools/tilebench.py 1024 2048 --types 4,0,3 --versions 5 --streams 10 > gpurun_out/tb59_p$p.log 2>&1
  VS_TCF_PAIR=$p timeout 300 python tools/tilebench.py 1024 --types 4 --versions 5 --streams 1 >> gpurun_out/tb59_p$p.log 2>&1
  VS_TCF_PAIR=$p timeout 400 python bench.py --no-e2e --no-cpu --dump-log gpurun_out/b59_p$p.json > gpurun_out/b59_p$p.log 2>&1
done
