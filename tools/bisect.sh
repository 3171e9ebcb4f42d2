#!/bin/bash
timeout 600 compute-sanitizer --tool memcheck --print-limit 3 python tools/one.py B xstat 2>&1 | grep -v "^=========     " | head -60
