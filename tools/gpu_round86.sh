#!/bin/bash
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 300 python -m pytest tests/test_gpu_tiles.py -q -p no:cacheprovider -k "53bit or 4096" > gpurun_out/t86.log 2>&1; echo "exit $?" >> gpurun_out/t86.log
