#!/bin/bash
# tcf v2 + epilogue with C_in loads one round ahead (overlapping the TMEM read-out)
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build68.log 2>&1
timeout 300 python -m pytest tests/test_gpu_tiles.py -q -p no:cacheprovider -x > gpurun_out/t68_tiles.log 2>&1; echo "exit $?" >> gpurun_out/t68_tiles.log
timeout 300 python -m pytest tests/test_gpu_runtime.py -q -p no:cacheprovider -x > gpurun_out/t68_rt.log 2>&1; echo "exit $?" >> gpurun_out/t68_rt.log
timeout 300 python tools/tilebench.py 1024 2048 --types 4,0,3 --versions 5 --streams 10 > gpurun_out/tb68.log 2>&1
timeout 300 python tools/tilebench.py 1024 --types 4 --versions 5 --streams 1 >> gpurun_out/tb68.log 2>&1
timeout 400 python bench.py --steps 5 --warmup 3 --no-e2e --no-cpu --dump-log gpurun_out/b68.json > gpurun_out/b68.log 2>&1
