#!/bin/bash
# critical-path streams only while idle: matmul alone / Cholesky alone / both
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build70.log 2>&1
timeout 400 python -m pytest tests/test_gpu_runtime.py tests/test_gpu_cfg5.py -q -p no:cacheprovider -x > gpurun_out/t70.log 2>&1; echo "exit $?" >> gpurun_out/t70.log
timeout 400 python bench.py --steps 5 --warmup 3 --no-e2e --no-cpu --only mm --dump-log gpurun_out/b70_mm.json > gpurun_out/b70_mm.log 2>&1
timeout 400 python bench.py --steps 5 --warmup 3 --no-e2e --no-cpu --only ch --dump-log gpurun_out/b70_ch.json > gpurun_out/b70_ch.log 2>&1
timeout 400 python bench.py --steps 5 --warmup 3 --no-e2e --no-cpu --dump-log gpurun_out/b70.json > gpurun_out/b70.log 2>&1
