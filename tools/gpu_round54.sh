#!/bin/bash
# cfg5 convergence sweep + its GPU test
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 600 python -m pytest tests/test_gpu_cfg5.py -q -p no:cacheprovider -x > gpurun_out/t54.log 2>&1; echo "exit $?" >> gpurun_out/t54.log
timeout 900 python tools/sweep_cfg5.py --out gpurun_out/cfg5.json > gpurun_out/cfg5.log 2>&1; echo "exit $?" >> gpurun_out/cfg5.log
