#!/bin/bash
# tcf v4: M-half double-buffered TMEM (N=256 MMAs), A-role/B-role split forms, B multicast pairs
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build67.log 2>&1
timeout 300 python -m pytest tests/test_gpu_tiles.py -q -p no:cacheprovider -x > gpurun_out/t67_tiles.log 2>&1; echo "exit $?" >> gpurun_out/t67_tiles.log
timeout 300 python -m pytest tests/test_gpu_runtime.py -q -p no:cacheprovider -x > gpurun_out/t67_rt.log 2>&1; echo "exit $?" >> gpurun_out/t67_rt.log
timeout 300 python tools/tilebench.py 1024 2048 --types 4,0,3 --versions 5 --streams 10 > gpurun_out/tb67.log 2>&1
timeout 300 python tools/tilebench.py 1024 --types 4 --versions 5 --streams 1 >> gpurun_out/tb67.log 2>&1
timeout 400 python bench.py --steps 5 --warmup 3 --no-e2e --no-cpu --dump-log gpurun_out/b67.json > gpurun_out/b67.log 2>&1
