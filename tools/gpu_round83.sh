#!/bin/bash
# K-chunked tensor-core accumulation: accuracy probe, tile + runtime tests, tilebench, bench
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build83.log 2>&1
timeout 600 python tools/acc_probe.py > gpurun_out/acc83.log 2>&1
timeout 600 python -m pytest tests/test_gpu_tiles.py tests/test_gpu_runtime.py tests/test_gpu_cfg5.py -q -p no:cacheprovider > gpurun_out/t83.log 2>&1; echo "exit $?" >> gpurun_out/t83.log
timeout 300 python tools/tilebench.py 1024 2048 --types 4,0 --versions 1,5 --streams 10 > gpurun_out/tb83.log 2>&1
timeout 400 python bench.py --steps 5 --warmup 3 --no-e2e --no-cpu > gpurun_out/b83.log 2>&1
