#!/bin/bash
timeout 300 python -X faulthandler tools/dbg_exchange.py c1:262144:262151 c3:65536:262144 dup:5000:7000 2>&1 | tail -8
timeout 900 python -m pytest tests/test_gpu_exchange.py tests/test_gpu_coprocess.py -m gpu -q -x 2>&1 | tail -3
