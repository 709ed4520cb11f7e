#!/bin/bash
# NN producer remap check + slot sweep + trsm/potrf launch breakdown
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 300 python -m pytest tests/test_gpu_tiles.py -q -p no:cacheprovider -x > gpurun_out/tiles.log 2>&1; echo "tiles exit $?" >> gpurun_out/tiles.log
timeout 300 python tools/tilebench.py 1024 --streams 1 --types 0,4 --versions 1 > gpurun_out/tilebench.log 2>&1
timeout 300 python tools/tilebench.py 1024 --streams 4 --types 0,4,2 --versions 1 >> gpurun_out/tilebench.log 2>&1
timeout 300 python tools/tilebench.py 1024 --streams 8 --types 0,4,2 --versions 1 >> gpurun_out/tilebench.log 2>&1
timeout 300 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/trsm_launches.csv python tools/tilebench.py 1024 --streams 1 --types 2,1 --versions 1 --iters 1 > gpurun_out/ncu_trsm.log 2>&1
for s in 4 6 8; do
  timeout 400 python bench.py --steps 3 --warmup 3 --slots $s > gpurun_out/bench_slots$s.log 2>&1
done
