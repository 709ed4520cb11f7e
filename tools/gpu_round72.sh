#!/bin/bash
# eager write-back: runtime tests (host data), bench with e2e
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build72.log 2>&1
timeout 400 python -m pytest tests/test_gpu_runtime.py tests/test_gpu_dist.py -q -p no:cacheprovider -x > gpurun_out/t72.log 2>&1; echo "exit $?" >> gpurun_out/t72.log
timeout 600 python bench.py --steps 5 --warmup 3 --no-cpu > gpurun_out/b72.log 2>&1
