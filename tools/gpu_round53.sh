#!/bin/bash
# session-3 re-validation: gpu tests, smoke, default bench, launch list
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build53.log 2>&1
timeout 900 python -m pytest tests -m gpu -q -p no:cacheprovider -x > gpurun_out/t53.log 2>&1; echo "exit $?" >> gpurun_out/t53.log
timeout 300 python __graft_entry__.py smoke > gpurun_out/smoke53.log 2>&1; echo "exit $?" >> gpurun_out/smoke53.log
timeout 900 python bench.py --dump-log gpurun_out/b53.json > gpurun_out/b53.log 2>&1
timeout 600 python bench.py --impl reference --steps 1 --warmup 0 > gpurun_out/ref53.log 2>&1
