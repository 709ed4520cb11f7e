#!/bin/bash
# full validation of the current state: gpu tests, smoke, default bench, reference arm
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build84.log 2>&1
timeout 900 python -m pytest tests -m gpu -q -p no:cacheprovider -x > gpurun_out/t84.log 2>&1; echo "exit $?" >> gpurun_out/t84.log
timeout 300 python __graft_entry__.py smoke > gpurun_out/smoke84.log 2>&1; echo "exit $?" >> gpurun_out/smoke84.log
timeout 900 python bench.py --dump-log gpurun_out/b84.json > gpurun_out/b84.log 2>&1
timeout 600 python bench.py --impl reference --steps 2 --warmup 1 > gpurun_out/ref84.log 2>&1
