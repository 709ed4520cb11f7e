#!/bin/bash
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 300 python -m pytest tests/test_gpu_runtime.py -q -p no:cacheprovider -k "b2048" > gpurun_out/t90.log 2>&1; echo "exit $?" >> gpurun_out/t90.log
