#!/bin/bash
# GPU tests + default bench (group_hold, 12 slots) with log
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 900 python -m pytest tests -m gpu -q -p no:cacheprovider -x > gpurun_out/t57.log 2>&1; echo "exit $?" >> gpurun_out/t57.log
timeout 900 python bench.py --dump-log gpurun_out/b57.json > gpurun_out/b57.log 2>&1
