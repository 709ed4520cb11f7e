#!/bin/bash
# tcf v2 + direct-store epilogue (16x256b TMEM fragments, no smem staging)
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build75.log 2>&1
timeout 300 python -m pytest tests/test_gpu_tiles.py -q -p no:cacheprovider -x > gpurun_out/t75_tiles.log 2>&1; echo "exit $?" >> gpurun_out/t75_tiles.log
timeout 300 python -m pytest tests/test_gpu_runtime.py -q -p no:cacheprovider -x > gpurun_out/t75_rt.log 2>&1; echo "exit $?" >> gpurun_out/t75_rt.log
timeout 300 python tools/tilebench.py 1024 2048 --types 4,0,3 --versions 5 --streams 10 > gpurun_out/tb75.log 2>&1
timeout 300 python tools/tilebench.py 1024 --types 4 --versions 5 --streams 1 >> gpurun_out/tb75.log 2>&1
timeout 400 python bench.py --steps 5 --warmup 3 --no-e2e --no-cpu --dump-log gpurun_out/b75.json > gpurun_out/b75.log 2>&1
