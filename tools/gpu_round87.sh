#!/bin/bash
# windowed input prefetch for the e2e path: runtime tests with prefetch on, e2e with windows 0/4/8/16
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build87.log 2>&1
VS_PREFETCH=8 timeout 400 python -m pytest tests/test_gpu_runtime.py -q -p no:cacheprovider -x > gpurun_out/t87.log 2>&1; echo "exit $?" >> gpurun_out/t87.log
for w in 0 4 8 16; do
  VS_PREFETCH=$w timeout 600 python bench.py --steps 2 --warmup 3 --no-cpu > gpurun_out/b87_w$w.log 2>&1
done
