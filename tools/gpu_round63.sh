#!/bin/bash
# oz v3 (SW32 rows, 5 stages): tests + tilebench
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 300 python -m pytest tests/test_gpu_tiles.py -q -p no:cacheprovider > gpurun_out/t63_tiles.log 2>&1; echo "exit $?" >> gpurun_out/t63_tiles.log
timeout 300 python -m pytest tests/test_gpu_runtime.py -q -p no:cacheprovider -k f64 > gpurun_out/t63_rt.log 2>&1; echo "exit $?" >> gpurun_out/t63_rt.log
timeout 300 python tools/tilebench.py 512 1024 2048 --types 0,4,3 --versions 6 --streams 1 > gpurun_out/tb63.log 2>&1
timeout 300 python tools/tilebench.py 1024 2048 --types 0 --versions 6 --streams 8 >> gpurun_out/tb63.log 2>&1
