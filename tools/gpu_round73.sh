#!/bin/bash
# input prefetch + eager write-back: runtime tests, e2e bench (prefetch on / off)
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build73.log 2>&1
timeout 400 python -m pytest tests/test_gpu_runtime.py -q -p no:cacheprovider -x > gpurun_out/t73.log 2>&1; echo "exit $?" >> gpurun_out/t73.log
timeout 600 python bench.py --steps 5 --warmup 3 --no-cpu > gpurun_out/b73.log 2>&1
VS_PREFETCH=0 timeout 600 python bench.py --steps 3 --warmup 3 --no-cpu > gpurun_out/b73_nopf.log 2>&1
